#!/bin/bash
# every 8(a)/8(f) row's kernel timed on its workload + ncu captures of the new kernels
mkdir -p gpurun_out
timeout 900 python tools/bench_idioms.py > gpurun_out/rows.jsonl 2> gpurun_out/rows.err
timeout 300 ncu --set full --clock-control none --import-source on -k regex:k_stencil27 -s 3 -c 1 -o gpurun_out/prof_stencil_async -f python tools/bench_idioms.py --no-cpu --reps 1 stencil256 > /dev/null 2>&1
timeout 300 ncu --set full --clock-control none --import-source on -k regex:k_spmv_jds -s 3 -c 1 -o gpurun_out/prof_jds64 -f python tools/bench_idioms.py --no-cpu --reps 1 jds_parboil > /dev/null 2>&1
timeout 300 ncu --set full --clock-control none --import-source on -k regex:k_cgcg -s 30 -c 1 -o gpurun_out/prof_cgcg -f python bench.py --steps 2 --warmup 3 --no-cpu > /dev/null 2>&1
cut -c1-220 gpurun_out/rows.jsonl
