# PDL on the textbook chain too; proxy tables after PDL; standalone P=8 SpMV timeline
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02s; mkdir -p $O
timeout 1200 python -m pytest tests/test_gpu_cg.py tests/test_gpu_cgcg.py tests/test_gpu_dist.py tests/test_gpu_p2p_mp.py -q -x > $O/pytest.log 2>&1; echo "rc=$?" >> $O/pytest.log
timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/bench.json 2> $O/bench.err
timeout 900 python tools/proxy_ranks.py --variant cgcg > $O/proxy_cgcg.jsonl 2> $O/proxy_cgcg.err
for P in 1 8; do XT_NOFLUSH=1 XT_REPS=10 timeout 300 python tools/xplan_times.py C $P 0 >> $O/xplan_times_noflush.txt 2>&1; done
XT_NOFLUSH=1 XT_REPS=10 timeout 300 python tools/xplan_times.py B 1 0 >> $O/xplan_times_noflush.txt 2>&1
