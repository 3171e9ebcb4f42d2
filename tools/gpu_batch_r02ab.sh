# parallel-round bank spreading: parity, create time (launch list), SpMV time, shared-memory conflicts
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02ab; mkdir -p $O
timeout 1500 python -m pytest tests/test_gpu_spmv.py tests/test_gpu_bounds.py tests/test_gpu_persist.py tests/test_gpu_cgcg.py tests/test_gpu_launch_modes.py -q -x > $O/pytest.log 2>&1; echo "rc=$?" >> $O/pytest.log
timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/bench.json 2> $O/bench.err
for c in C B; do timeout 300 python tools/gap.py $c rand >> $O/gap.txt 2>&1; done
timeout 900 python tools/proxy_ranks.py --variant cgcg --ps 8 --ranks first > $O/proxy8.jsonl 2> $O/proxy8.err
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file $O/launches.csv python bench.py --steps 2 --warmup 3 --no-cpu > /dev/null 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_spmv_xplan -s 30 -c 1 -o $O/xplan_cg python bench.py --steps 1 --warmup 3 --no-cpu > /dev/null 2>&1
