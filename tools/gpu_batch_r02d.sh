cd $GRAFT_REPO_ROOT
O=gpurun_out/r02d; mkdir -p $O
timeout 900 python bench.py --steps 20 --warmup 5 > $O/bench.json 2> $O/bench.err
for v in cgcg persist; do
  timeout 900 python tools/proxy_ranks.py --kernel xplan --steps 10 --variant $v > $O/proxy_$v.jsonl 2> $O/proxy_$v.err
done
for tr in p2p nccl; do
  SPMV_BENCH_FORCE_DIST=1 SPMV_TRANSPORT=$tr timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 \
    --master-addr 127.0.0.1 --master-port 29555 bench.py --steps 10 --warmup 3 --no-cpu > $O/bench_dist1_$tr.json 2> $O/bench_dist1_$tr.err
done
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file $O/launches.csv python bench.py --steps 2 --warmup 3 --no-cpu > /dev/null 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_spmv_xplan -s 30 -c 1 -o $O/xplan_cg python bench.py --steps 1 --warmup 3 --no-cpu > /dev/null 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_cg_persist -s 0 -c 1 -o $O/persist python bench.py --steps 1 --warmup 3 --no-cpu --cg-variant persist > /dev/null 2>&1
timeout 3000 python -m pytest tests -m gpu -q -x > $O/pytest_gpu.log 2>&1
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > $O/smoke.log 2>&1
