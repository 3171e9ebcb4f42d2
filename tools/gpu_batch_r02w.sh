# PDL on the p2p path too: 2-process p2p tests + one-rank transports vs single GPU (same box)
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02w; mkdir -p $O
timeout 1200 python -m pytest tests/test_gpu_p2p_mp.py tests/test_gpu_dist.py tests/test_gpu_cgcg.py -q -x > $O/pytest.log 2>&1; echo "rc=$?" >> $O/pytest.log
timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/bench_single.json 2> $O/bench_single.err
for T in nccl p2p; do
  SPMV_BENCH_FORCE_DIST=1 SPMV_TRANSPORT=$T timeout 900 python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 \
    --master-addr 127.0.0.1 --master-port 29557 bench.py --steps 20 --warmup 5 --no-cpu > $O/bench_dist1_$T.json 2> $O/bench_dist1_$T.err
  SPMV_PDL=0 SPMV_BENCH_FORCE_DIST=1 SPMV_TRANSPORT=$T timeout 900 python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 \
    --master-addr 127.0.0.1 --master-port 29558 bench.py --steps 20 --warmup 5 --no-cpu > $O/bench_dist1_${T}_nopdl.json 2> $O/bench_dist1_${T}_nopdl.err
done
XT_NOFLUSH=1 XT_REPS=10 timeout 300 python tools/xplan_times.py C 8 0 >> $O/xplan_times_noflush.txt 2>&1
XT_NOFLUSH=1 XT_REPS=10 timeout 300 python tools/xplan_times.py C 4 0 >> $O/xplan_times_noflush.txt 2>&1
