cd $GRAFT_REPO_ROOT
O=gpurun_out/r02e; mkdir -p $O
SPMV_BENCH_FORCE_DIST=1 SPMV_TRANSPORT=p2p timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 \
    --master-addr 127.0.0.1 --master-port 29555 bench.py --steps 10 --warmup 3 --no-cpu > $O/bench_dist1_p2p.json 2> $O/bench_dist1_p2p.err
for i in 1 2 3; do XT_PER_CLUSTER=1 timeout 120 python tools/xplan_times.py C 1 0 >> $O/cluster_times.txt 2>&1; done
timeout 300 python -m pytest tests/test_gpu_persist.py tests/test_gpu_p2p_mp.py -q -x > $O/pytest.log 2>&1
