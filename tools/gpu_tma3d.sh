#!/bin/bash
# 3-D TMA tile-load check (tools/microbench/tma3d.cu) for several boxes / origins
mkdir -p gpurun_out
for a in "66 18 -2 -1 0" "66 18 -2 0 0" "66 18 0 -1 0" "66 18 254 254 0" "66 18 -2 -1 1"; do
  timeout 30 tools/microbench/tma3d $a >> gpurun_out/tma3d.txt 2>&1
done
cat gpurun_out/tma3d.txt
