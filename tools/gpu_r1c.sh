#!/bin/bash
# bench + ncu full captures of the Parboil merge kernel and the stencil SELL kernel + XPLAN per-CTA times
mkdir -p gpurun_out
timeout 600 python bench.py --steps 10 --warmup 3 > gpurun_out/bench.json 2> gpurun_out/bench.err; cat gpurun_out/bench.json
timeout 300 python tools/one.py C xplan SPMV_XPLAN_TIMES=1 > gpurun_out/xplan_times_C.txt 2>&1
timeout 300 python tools/one.py B xplan SPMV_XPLAN_TIMES=1 > gpurun_out/xplan_times_B.txt 2>&1
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_spmv_merge -s 2 -c 1 \
   -o gpurun_out/prof_parboil_merge -f python tools/one.py parboil merge > gpurun_out/prof_parboil.log 2>&1; echo "ncu parboil $?"
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_spmv_sell -s 2 -c 1 \
   -o gpurun_out/prof_stencil_sell -f python tools/one.py stencil256 sell > gpurun_out/prof_stencil.log 2>&1; echo "ncu stencil $?"
