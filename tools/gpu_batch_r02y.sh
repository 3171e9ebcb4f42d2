# probe: how much of the P = 8 / P = 4 block SpMV is the paired warps' second chunk?
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02y; mkdir -p $O
for P in 8 4; do
  XT_NOFLUSH=1 XT_REPS=10 timeout 300 python tools/xplan_times.py C $P 0 >> $O/times.txt 2>&1
  echo "nopair probe" >> $O/times.txt
  SPMV_LIB_PATH=tools/variants/lib_nopair.so XT_NOFLUSH=1 XT_REPS=10 timeout 300 python tools/xplan_times.py C $P 0 >> $O/times.txt 2>&1
done
