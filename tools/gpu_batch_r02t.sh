# x bulk copy ahead of the plan's L2 prefetch in the TMA queue; per-cluster streaming ends
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02t; mkdir -p $O
timeout 1200 python -m pytest tests/test_gpu_spmv.py tests/test_gpu_persist.py tests/test_gpu_cgcg.py -q -x -k "xplan or persist or cgcg or full" > $O/pytest.log 2>&1; echo "rc=$?" >> $O/pytest.log
for P in 1 4 8; do XT_NOFLUSH=1 XT_REPS=10 timeout 300 python tools/xplan_times.py C $P 0 >> $O/xplan_times_noflush.txt 2>&1; done
XT_NOFLUSH=1 XT_REPS=6 XT_PER_CLUSTER=1 timeout 300 python tools/xplan_times.py C 1 0 >> $O/xplan_per_cluster.txt 2>&1
timeout 900 python tools/proxy_ranks.py --variant cgcg > $O/proxy_cgcg.jsonl 2> $O/proxy_cgcg.err
timeout 900 python tools/proxy_ranks.py --variant persist > $O/proxy_persist.jsonl 2> $O/proxy_persist.err
timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/bench.json 2> $O/bench.err
