cd $GRAFT_REPO_ROOT
O=gpurun_out/r02i; mkdir -p $O
T() { timeout 120 python tools/time_one.py "$@" >> $O/times.jsonl 2>>$O/times.err; }
for m in B C A W S; do
  T ${m}_steady $m xplan TIME_STEADY=1
  T ${m}_steady_cpw1 $m xplan TIME_STEADY=1 SPMV_LIB_PATH=tools/variants/lib_cpw1.so
done
T B_steady_B8 B xplan TIME_STEADY=1 SPMV_XPLAN_B=8
T B_steady_B8_cpw1 B xplan TIME_STEADY=1 SPMV_XPLAN_B=8 SPMV_LIB_PATH=tools/variants/lib_cpw1.so
SPMV_LIB_PATH=tools/variants/lib_cpw1.so timeout 900 python tools/proxy_ranks.py --kernel xplan --steps 10 --variant persist --ranks first > $O/proxy_persist_cpw1.jsonl 2> $O/proxy_cpw1.err
