#!/bin/bash
# stencil GPU tests, TMA vs cp.async timing on 256^3, z-chunk sweep, build variants, ncu of the TMA kernel
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_stencil.py -x -q > gpurun_out/pytest_stencil.log 2>&1; echo "exit $?" >> gpurun_out/pytest_stencil.log
for i in 1 2; do
  timeout 120 python tools/time_stencil.py tma 256 >> gpurun_out/st.jsonl 2>&1
  timeout 120 python tools/time_stencil.py cpasync 256 SPMV_STENCIL_TMA=0 >> gpurun_out/st.jsonl 2>&1
done
for zc in 9 13 26; do timeout 120 python tools/time_stencil.py tma_z$zc 256 SPMV_STENCIL_ZCHUNK=$zc >> gpurun_out/st.jsonl 2>&1; done
ls tools/variants/*.so > /dev/null 2>&1 && bash tools/run_stencil_variants.sh >> gpurun_out/st.jsonl 2>&1
timeout 300 ncu --set full --clock-control none --import-source on -k regex:k_stencil27 -s 3 -c 1 -o gpurun_out/prof_stencil_tma -f python tools/time_stencil.py x 256 > /dev/null 2>&1
tail -3 gpurun_out/pytest_stencil.log; grep '"us"' gpurun_out/st.jsonl
