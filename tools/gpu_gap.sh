#!/bin/bash
O=gpurun_out/gap; mkdir -p $O
for c in C B; do for xk in ones rand; do timeout 120 python tools/gap.py $c $xk >> $O/gap.txt 2>&1; done; done
for i in 1 2; do XT_NOFLUSH=1 XT_REPS=20 timeout 120 python tools/xplan_times.py B 1 0 | tail -1 >> $O/gap.txt 2>&1; done
cat $O/gap.txt
