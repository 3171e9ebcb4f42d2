# p2p: per-CTA partial pushes (no last-CTA reduction); 2-process tests + one-rank transports
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02aa; mkdir -p $O
timeout 1200 python -m pytest tests/test_gpu_p2p_mp.py tests/test_gpu_dist.py tests/test_gpu_cgcg.py tests/test_gpu_cg.py tests/test_gpu_launch_modes.py -q -x > $O/pytest.log 2>&1; echo "rc=$?" >> $O/pytest.log
timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/bench_single.json 2> $O/bench_single.err
for T in p2p nccl; do
  SPMV_BENCH_FORCE_DIST=1 SPMV_TRANSPORT=$T timeout 900 python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 \
    --master-addr 127.0.0.1 --master-port 29559 bench.py --steps 20 --warmup 5 --no-cpu > $O/bench_dist1_$T.json 2> $O/bench_dist1_$T.err
done
SPMV_BENCH_FORCE_DIST=1 SPMV_TRANSPORT=p2p timeout 600 ncu --target-processes all --metrics gpu__time_duration.sum --clock-control none -c 300 --csv --log-file $O/p2p_launches.csv \
  python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 --master-addr 127.0.0.1 --master-port 29560 bench.py --steps 2 --warmup 3 --no-cpu > /dev/null 2>&1
