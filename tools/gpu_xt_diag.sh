cd $GRAFT_REPO_ROOT
O=gpurun_out/xtdiag; mkdir -p $O
T() { timeout 120 python tools/time_one.py "$@" >> $O/times.jsonl 2>>$O/times.err; }
for cfg in "" "SPMV_XT_B=8" "SPMV_XT_NS=4"; do
T "xt_C $cfg" C xt $cfg
T "noproc_C $cfg" C xt SPMV_LIB_PATH=tools/variants/lib_xtnoproc.so $cfg
T "nogather_C $cfg" C xt SPMV_LIB_PATH=tools/variants/lib_xtnogather.so $cfg
done
