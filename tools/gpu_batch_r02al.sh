cd $GRAFT_REPO_ROOT
O=gpurun_out/r02al; mkdir -p $O
timeout 1500 python -m pytest tests/test_gpu_spmv.py tests/test_gpu_bounds.py tests/test_gpu_launch_modes.py -q -x > $O/pytest.log 2>&1; echo "rc=$?" >> $O/pytest.log
timeout 600 python bench.py --steps 20 --warmup 5 --no-cpu > $O/bench.json 2> $O/bench.err
