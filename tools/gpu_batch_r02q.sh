# persistent CG with published partials (barrier + reduction in one round trip)
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02q; mkdir -p $O
timeout 900 python -m pytest tests/test_gpu_persist.py tests/test_gpu_cgcg.py -q -x > $O/pytest.log 2>&1; echo "rc=$?" >> $O/pytest.log
for P in 1 8; do timeout 300 python tools/persist_times.py C $P 0 >> $O/persist_times.txt 2>&1; done
timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/bench.json 2> $O/bench.err
timeout 900 python tools/proxy_ranks.py --variant persist > $O/proxy_persist.jsonl 2> $O/proxy_persist.err
timeout 900 python tools/proxy_ranks.py --variant cgcg > $O/proxy_cgcg.jsonl 2> $O/proxy_cgcg.err
