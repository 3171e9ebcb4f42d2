# persistent CG: stashed update rows, pre-barrier gamma sums, cluster-aggregated barrier option; bank-conflict-free probe
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02m; mkdir -p $O
timeout 900 python -m pytest tests/test_gpu_persist.py tests/test_gpu_cgcg.py -q -x > $O/pytest.log 2>&1; echo "rc=$?" >> $O/pytest.log
for P in 1 8; do
  for BM in 0 1; do echo "bar_mode=$BM" >> $O/persist_times.txt; SPMV_PERSIST_BAR=$BM timeout 300 python tools/persist_times.py C $P 0 >> $O/persist_times.txt 2>&1; done
  echo "noconf probe" >> $O/persist_times.txt; SPMV_LIB_PATH=tools/variants/lib_noconf.so timeout 300 python tools/persist_times.py C $P 0 >> $O/persist_times.txt 2>&1
done
timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/bench.json 2> $O/bench.err
timeout 600 python tools/proxy_ranks.py --variant persist > $O/proxy_persist.jsonl 2> $O/proxy.err
