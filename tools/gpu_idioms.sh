#!/bin/bash
# One gpurun call for the NEXT-4 idioms: GPU parity tests, timings, fp64 peak
# microbenchmark, ncu captures of the idiom kernels.  Outputs in gpurun_out/.
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_idioms.py -x -q > gpurun_out/pytest_idioms.log 2>&1
echo "pytest exit $?" >> gpurun_out/pytest_idioms.log
[ -x tools/microbench/dfma ] || nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o tools/microbench/dfma tools/microbench/dfma.cu
tools/microbench/dfma > gpurun_out/dfma.json 2>&1
timeout 600 python tools/bench_idioms.py > gpurun_out/idioms.jsonl 2> gpurun_out/idioms.err
if [ -n "$NCU" ]; then
  timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_ep -s 3 -c 1 \
     -o gpurun_out/prof_ep -f python tools/bench_idioms.py --no-cpu --reps 1 ep_C > gpurun_out/ncu_ep.log 2>&1
  timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_hist -s 3 -c 1 \
     -o gpurun_out/prof_is -f python tools/bench_idioms.py --no-cpu --reps 1 is_C > gpurun_out/ncu_is.log 2>&1
  timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_reduce -s 3 -c 1 \
     -o gpurun_out/prof_dot -f python tools/bench_idioms.py --no-cpu --reps 1 dot_2p27 > gpurun_out/ncu_dot.log 2>&1
fi
tail -3 gpurun_out/pytest_idioms.log
cat gpurun_out/dfma.json gpurun_out/idioms.jsonl
