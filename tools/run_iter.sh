for m in C B; do timeout 60 python tools/time_one.py b16 $m xplan SPMV_XPLAN_B=16; timeout 60 python tools/one.py $m xplan SPMV_XPLAN_B=16 2>&1 | grep -o "'grid': [0-9]*"; done
