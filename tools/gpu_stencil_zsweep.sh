#!/bin/bash
# z-chunk sweep of the default (TMA) stencil on 256^3, 3 repeats each
mkdir -p gpurun_out
for i in 1 2 3; do for zc in 11 12 13 14 15 16 18; do
  timeout 60 python tools/time_stencil.py z$zc 256 SPMV_STENCIL_ZCHUNK=$zc >> gpurun_out/zs.jsonl 2>&1
done; done
cat gpurun_out/zs.jsonl
