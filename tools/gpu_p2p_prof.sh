#!/bin/bash
# p2p transport at one rank: bench line + ncu launch list (per-kernel device times)
O=gpurun_out/p2p; mkdir -p $O
SPMV_BENCH_FORCE_DIST=1 SPMV_TRANSPORT=p2p timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 \
    --master-addr 127.0.0.1 --master-port 29555 bench.py --steps 10 --warmup 3 --no-cpu > $O/bench_dist1_p2p.json 2> $O/bench_dist1_p2p.err
timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu > $O/bench_single.json 2> $O/bench_single.err
SPMV_BENCH_FORCE_DIST=1 SPMV_TRANSPORT=p2p timeout 900 ncu --target-processes all --metrics gpu__time_duration.sum --clock-control none -c 600 --csv \
   --log-file $O/p2p_launches.csv python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 \
    --master-addr 127.0.0.1 --master-port 29556 bench.py --steps 2 --warmup 3 --no-cpu > $O/ncu_bench.log 2>&1
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 600 --csv \
   --log-file $O/single_launches.csv python bench.py --steps 2 --warmup 3 --no-cpu > $O/ncu_single.log 2>&1
python tools/launch_shares.py $O/p2p_launches.csv > $O/p2p_shares.txt 2>&1
python tools/launch_shares.py $O/single_launches.csv > $O/single_shares.txt 2>&1
tail -c 600 $O/bench_dist1_p2p.json; tail -c 600 $O/bench_single.json; head -12 $O/p2p_shares.txt; head -12 $O/single_shares.txt
