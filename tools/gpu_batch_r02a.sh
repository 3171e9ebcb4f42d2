# round-2 batch: sanitizer tier, proxy table, transports, l2 window, bench with CPU baselines
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02a; mkdir -p $O
S=/usr/local/cuda/bin/compute-sanitizer
for tool in memcheck racecheck synccheck; do
  timeout 1200 $S --tool $tool --print-limit 20 python tools/sanitize_cases.py > $O/sanitizer_$tool.log 2>&1
  echo "rc=$?" >> $O/sanitizer_$tool.log
done
timeout 900 python tools/proxy_ranks.py --kernel xplan --steps 10 > $O/proxy_xplan.jsonl 2> $O/proxy_xplan.err
# 1-rank transports (torchrun with one rank; the row-sharded path with p2p / nccl) and the single-GPU path
for tr in p2p nccl; do
  SPMV_BENCH_FORCE_DIST=1 SPMV_TRANSPORT=$tr timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 \
    --master-addr 127.0.0.1 --master-port 29555 bench.py --steps 10 --warmup 3 --no-cpu > $O/bench_dist1_$tr.json 2> $O/bench_dist1_$tr.err
done
T() { timeout 120 python tools/time_one.py "$@" >> $O/times.jsonl 2>>$O/times.err; }
T parboil_sellsort parboil sellsort
T parboil_sellsort_l2w parboil sellsort TIME_L2W=1
T parboil_merge parboil merge
T parboil_merge_l2w parboil merge TIME_L2W=1
T parboil_vector parboil vector
T parboil_vector_l2w parboil vector TIME_L2W=1
T C_xplan C xplan
timeout 900 python bench.py --steps 20 --warmup 5 > $O/bench.json 2> $O/bench.err
timeout 1500 python -m pytest tests/test_gpu_spmv.py -x -q -k "xplan or l2_window" > $O/pytest_spmv.log 2>&1
