timeout 300 python -m pytest tests/test_gpu_spmv.py tests/test_gpu_cg.py tests/test_gpu_dist.py -x -q -k "xplan or nas or npb or parboil or dist" > gpurun_out/pytest_gpu.log 2>&1; echo "pytest exit $?" >> gpurun_out/pytest_gpu.log; tail -2 gpurun_out/pytest_gpu.log; grep -E "^E " gpurun_out/pytest_gpu.log | head -5
for m in C B; do timeout 60 python tools/time_one.py v5 $m xplan; done
timeout 300 python bench.py --steps 10 --warmup 3 --no-cpu > gpurun_out/bench.json 2> gpurun_out/bench.err; cut -c1-300 gpurun_out/bench.json
bash tools/gpu_prof.sh xplanC C xplan
