cd $GRAFT_REPO_ROOT
O=gpurun_out/r02h; mkdir -p $O
for v in cgcg persist; do
  timeout 900 python tools/proxy_ranks.py --kernel xplan --steps 10 --variant $v --ranks first,last > $O/proxy_$v.jsonl 2> $O/proxy_$v.err
done
timeout 600 python -m pytest tests/test_gpu_persist.py tests/test_gpu_cgcg.py -q -x > $O/pytest.log 2>&1
T() { timeout 120 python tools/time_one.py "$@" >> $O/times.jsonl 2>>$O/times.err; }
T A A xplan
T S S xplan
T W W xplan
