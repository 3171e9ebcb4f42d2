cd $GRAFT_REPO_ROOT
O=gpurun_out/r02at; mkdir -p $O
timeout 1200 python -m pytest tests/test_gpu_bounds.py -q > $O/pytest.log 2>&1; echo "rc=$?" >> $O/pytest.log
