# bank-spread plan: full GPU suite, smoke, bench, proxy tables, launch list, ncu of the SpMV in CG
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02o; mkdir -p $O
timeout 2400 python -m pytest tests -m gpu -q > $O/pytest_gpu.log 2>&1; echo "rc=$?" >> $O/pytest_gpu.log
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > $O/smoke.log 2>&1; echo "rc=$?" >> $O/smoke.log
timeout 900 python bench.py --steps 20 --warmup 5 > $O/bench.json 2> $O/bench.err
timeout 900 python tools/proxy_ranks.py --variant cgcg > $O/proxy_cgcg.jsonl 2> $O/proxy_cgcg.err
timeout 900 python tools/proxy_ranks.py --variant persist > $O/proxy_persist.jsonl 2> $O/proxy_persist.err
for P in 1 2 4 8; do timeout 300 python tools/persist_times.py C $P 0 >> $O/persist_times.txt 2>&1; done
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file $O/launches.csv python bench.py --steps 2 --warmup 3 --no-cpu > /dev/null 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_spmv_xplan -s 30 -c 1 -o $O/xplan_cg python bench.py --steps 1 --warmup 3 --no-cpu > /dev/null 2>&1
_PT_CHILD=1 timeout 600 ncu --set full --clock-control none -k regex:k_cg_persist -c 1 -o $O/persist_P8 python tools/persist_times.py C 8 0 > /dev/null 2>&1
