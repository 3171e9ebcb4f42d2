cd $GRAFT_REPO_ROOT
O=gpurun_out/xtprof3; mkdir -p $O
L=SPMV_LIB_PATH=tools/variants/lib_xtprof.so
timeout 120 python tools/xt_case.py C $L > $O/c_b2.txt 2>&1
T() { timeout 120 python tools/time_one.py "$@" >> $O/times.jsonl 2>>$O/times.err; }
T xt_C C xt
T xt_C_dyn0 C xt SPMV_XT_DYN=0
T xt_C_B4 C xt SPMV_XT_B=4
T xt_C_B8 C xt SPMV_XT_B=8
T xt_C_NS5 C xt SPMV_XT_NS=5
T xt_C_NS9 C xt SPMV_XT_NS=9
T xt_B B xt
T xt_B_B8 B xt SPMV_XT_B=8
T xplan_C C xplan
timeout 900 python -m pytest tests/test_gpu_xt.py -x -q > $O/pytest_xt.log 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_spmv_xt -s 2 -c 1 -o $O/xt_C python tools/one.py C xt > $O/ncu_c.log 2>&1
