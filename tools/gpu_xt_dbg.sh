cd $GRAFT_REPO_ROOT
O=gpurun_out/xtdbg; mkdir -p $O
S=/usr/local/cuda/bin/compute-sanitizer
timeout 300 $S --tool memcheck --print-limit 8 python tools/xt_case.py powerlaw_small SPMV_XT_B=4 SPMV_XT_Q=2 > $O/pl_b4q2.txt 2>&1
timeout 120 python tools/xt_case.py C > $O/c.txt 2>&1
timeout 120 python tools/xt_case.py B > $O/b.txt 2>&1
bash tools/gpu_xt.sh
