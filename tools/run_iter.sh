for m in C B; do bash tools/run_variants.sh $m xplan; done
timeout 300 python -m pytest tests/test_gpu_spmv.py tests/test_gpu_cg.py -x -q -k "xplan or nas or npb" > gpurun_out/pytest_gpu.log 2>&1; echo "pytest exit $?" >> gpurun_out/pytest_gpu.log; tail -2 gpurun_out/pytest_gpu.log
