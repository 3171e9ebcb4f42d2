cd $GRAFT_REPO_ROOT
O=gpurun_out/r02b; mkdir -p $O
timeout 1500 python -m pytest tests/test_gpu_persist.py tests/test_gpu_xt.py tests/test_gpu_cgcg.py tests/test_gpu_cg.py -x -q > $O/pytest_a.log 2>&1
timeout 1200 python -m pytest tests/test_gpu_p2p_mp.py tests/test_gpu_dist.py tests/test_gpu_spmv.py -x -q > $O/pytest_b.log 2>&1
timeout 1800 python -m pytest tests/test_gpu_sanitizer.py -x -q > $O/pytest_san.log 2>&1
for a in "C 1 0" "C 8 0" "C 4 0" "B 1 0"; do timeout 120 python tools/xplan_times.py $a >> $O/xplan_times.txt 2>&1; done
timeout 900 python tools/proxy_ranks.py --kernel xplan --steps 10 --variant persist --ranks first > $O/proxy_persist.jsonl 2> $O/proxy_persist.err
for tr in p2p; do
  SPMV_BENCH_FORCE_DIST=1 SPMV_TRANSPORT=$tr timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 \
    --master-addr 127.0.0.1 --master-port 29555 bench.py --steps 10 --warmup 3 --no-cpu > $O/bench_dist1_$tr.json 2> $O/bench_dist1_$tr.err
done
timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/bench.json 2> $O/bench.err
