cd $GRAFT_REPO_ROOT
O=gpurun_out/r02k; mkdir -p $O
T() { timeout 150 python tools/time_one.py "$@" >> $O/times.jsonl 2>>$O/times.err; }
T parboil parboil sellsort
T parboil_steady parboil sellsort TIME_STEADY=1
for m in C B A W S; do T ${m}_steady $m xplan TIME_STEADY=1; done
for v in cgcg persist; do
  timeout 900 python tools/proxy_ranks.py --kernel xplan --steps 10 --variant $v --ranks first,last > $O/proxy_$v.jsonl 2> $O/proxy_$v.err
done
timeout 2400 python -m pytest tests -m gpu -q -x > $O/pytest_gpu.log 2>&1
