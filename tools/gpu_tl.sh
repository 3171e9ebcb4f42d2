#!/bin/bash
# XPLAN per-CTA timelines with SM ids (steady state), plus the p2p 1-rank bench after the unrolled last-CTA sum
O=gpurun_out/tl; mkdir -p $O; rm -f $O/dump_*.txt
for i in 1 2 3 4 5 6; do XT_NOFLUSH=1 XT_REPS=20 XT_DUMP=$O/dump_$i.txt XT_PER_CLUSTER=1 timeout 120 python tools/xplan_times.py C 1 0 | tail -1 >> $O/summary.txt 2>&1; done
SPMV_BENCH_FORCE_DIST=1 SPMV_TRANSPORT=p2p timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 \
    --master-addr 127.0.0.1 --master-port 29555 bench.py --steps 10 --warmup 3 --no-cpu > $O/bench_dist1_p2p.json 2> $O/bench_dist1_p2p.err
cat $O/summary.txt; tail -c 400 $O/bench_dist1_p2p.json
