cd $GRAFT_REPO_ROOT
O=gpurun_out/meta; mkdir -p $O
T() { timeout 150 python tools/time_one.py "$@" >> $O/times.jsonl 2>>$O/times.err; }
for rep in 1 2; do
for m in C B; do
  T ${m}_base $m xplan TIME_STEADY=1 SPMV_LIB_PATH=tools/variants/lib_base.so
  T ${m}_meta $m xplan TIME_STEADY=1
  T ${m}_meta_u8 $m xplan TIME_STEADY=1 SPMV_LIB_PATH=tools/variants/lib_u8.so
  T ${m}_meta_u7 $m xplan TIME_STEADY=1 SPMV_LIB_PATH=tools/variants/lib_u7.so
done
done
timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu > $O/bench.json 2> $O/bench.err
SPMV_LIB_PATH=tools/variants/lib_base.so timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu > $O/bench_base.json 2> $O/bench_base.err
timeout 600 python -m pytest tests/test_gpu_spmv.py -q -x -k "xplan or nas_full" > $O/pytest.log 2>&1
