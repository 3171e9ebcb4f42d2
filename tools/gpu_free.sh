cd $GRAFT_REPO_ROOT
O=gpurun_out/free; mkdir -p $O
timeout 900 python -m pytest tests/test_gpu_spmv.py tests/test_gpu_cgcg.py tests/test_gpu_p2p_mp.py -q -x -k "xplan or nas_full or npb or zeta or p2p or cgcg" > $O/pytest.log 2>&1
T() { timeout 150 python tools/time_one.py "$@" >> $O/times.jsonl 2>>$O/times.err; }
for rep in 1 2; do
for m in C B; do
  T ${m}_free $m xplan TIME_STEADY=1
  T ${m}_free_k4 $m xplan TIME_STEADY=1 SPMV_LIB_PATH=tools/variants/lib_free_k4.so
  T ${m}_nofree $m xplan TIME_STEADY=1 SPMV_LIB_PATH=tools/variants/lib_nofree.so
done
done
timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu > $O/bench.json 2> $O/bench.err
SPMV_LIB_PATH=tools/variants/lib_free_k4.so timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu > $O/bench_k4.json 2> $O/bench_k4.err
SPMV_LIB_PATH=tools/variants/lib_nofree.so timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu > $O/bench_nofree.json 2> $O/bench_nofree.err
