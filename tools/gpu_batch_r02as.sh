# per-kernel ncu cost of the p2p hooks at one rank (after per-CTA pushes + one publication in k_cgcg)
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02as; mkdir -p $O
SPMV_BENCH_FORCE_DIST=1 SPMV_TRANSPORT=p2p timeout 600 ncu --target-processes all --metrics gpu__time_duration.sum --clock-control none -c 300 --csv --log-file $O/p2p_launches.csv \
  python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 --master-addr 127.0.0.1 --master-port 29563 bench.py --steps 2 --warmup 3 --no-cpu > /dev/null 2>&1
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 300 --csv --log-file $O/single_launches.csv python bench.py --steps 2 --warmup 3 --no-cpu > /dev/null 2>&1
