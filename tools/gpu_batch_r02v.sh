# persisting-L2 window over small plans as the default: parity + proxy tables + bench
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02v; mkdir -p $O
timeout 1500 python -m pytest tests/test_gpu_spmv.py tests/test_gpu_persist.py tests/test_gpu_cgcg.py tests/test_gpu_cg.py tests/test_gpu_dist.py tests/test_gpu_bounds.py -q -x > $O/pytest.log 2>&1; echo "rc=$?" >> $O/pytest.log
timeout 900 python tools/proxy_ranks.py --variant cgcg > $O/proxy_cgcg.jsonl 2> $O/proxy_cgcg.err
timeout 900 python tools/proxy_ranks.py --variant persist > $O/proxy_persist.jsonl 2> $O/proxy_persist.err
timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/bench.json 2> $O/bench.err
for c in S W A B; do timeout 300 python tools/gap.py $c rand >> $O/gap.txt 2>&1; SPMV_XPLAN_PLANWIN=0 timeout 300 python tools/gap.py $c rand >> $O/gap_nowin.txt 2>&1; done
