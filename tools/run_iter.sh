timeout 600 python -m pytest tests/test_gpu_spmv.py -x -q -k "merge or parboil" > gpurun_out/pytest_gpu.log 2>&1; echo "pytest exit $?" >> gpurun_out/pytest_gpu.log; tail -2 gpurun_out/pytest_gpu.log
for k in merge; do timeout 60 python tools/time_one.py $k parboil $k; done
bash tools/gpu_prof.sh mergeP parboil merge
