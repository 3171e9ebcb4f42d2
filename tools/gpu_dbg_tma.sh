mkdir -p gpurun_out
for d in "64 16 3" "128 32 8" "2 3 5" "66 17 9"; do timeout 60 python tools/dbg_stencil_tma.py $d >> gpurun_out/dbg.txt 2>&1; done
grep -q "illegal" gpurun_out/dbg.txt && exit 1
bash tools/gpu_stencil_tma.sh
