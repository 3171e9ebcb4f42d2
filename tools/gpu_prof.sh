#!/bin/bash
# ncu full capture of one SpMV variant: tools/gpu_prof.sh NAME MATRIX KERNEL [ENV=VAL...]
name=$1; shift
mkdir -p gpurun_out
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_spmv -s 2 -c 1 \
   -o gpurun_out/prof_$name -f python tools/one.py "$@" > gpurun_out/prof_$name.log 2>&1
echo "ncu exit $?"
