#!/bin/bash
# XT kernel bring-up on the GPU box: smoke runs, parity tests, timings.
cd "$(dirname "$0")/.." || exit 1
O=gpurun_out/xt
mkdir -p $O
T() { timeout 120 python tools/time_one.py "$@" >> $O/times.jsonl 2>>$O/times.err; }
timeout 60 python tools/time_one.py xt_S S xt SPMV_DEBUG=1 > $O/first.txt 2>&1; echo "rc=$?" >> $O/first.txt
timeout 900 python -m pytest tests/test_gpu_xt.py -x -q -k "makea_S or laplace or multipiece or alpha_beta" > $O/pytest_quick.log 2>&1
T xt_C C xt
T xplan_C C xplan
T xt_B B xt
T xplan_B B xplan
T xt_C_B4 C xt SPMV_XT_B=4
T xt_C_B8 C xt SPMV_XT_B=8
T xt_C_NS5 C xt SPMV_XT_NS=5
T xt_C_NS9 C xt SPMV_XT_NS=9
T xt_B_B8 B xt SPMV_XT_B=8
timeout 1500 python -m pytest tests/test_gpu_xt.py -x -q > $O/pytest_xt.log 2>&1
