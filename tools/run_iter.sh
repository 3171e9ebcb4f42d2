timeout 300 python -m pytest tests/test_gpu_spmv.py tests/test_gpu_cg.py -x -q -k "xplan or nas or npb or parboil" > gpurun_out/pytest_gpu.log 2>&1; echo "pytest exit $?" >> gpurun_out/pytest_gpu.log; tail -3 gpurun_out/pytest_gpu.log
timeout 300 python tools/sweep.py C B > gpurun_out/sweep.jsonl 2> gpurun_out/sweep.err; grep -E "auto|xplan" gpurun_out/sweep.jsonl
timeout 300 python bench.py --steps 10 --warmup 3 --no-cpu > gpurun_out/bench.json 2> gpurun_out/bench.err; cut -c1-400 gpurun_out/bench.json
bash tools/gpu_prof.sh xplanC C xplan
