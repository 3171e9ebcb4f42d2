cd $GRAFT_REPO_ROOT
O=gpurun_out/r02ao; mkdir -p $O
timeout 1200 python -m pytest tests/test_bench_contract.py -q > $O/pytest.log 2>&1; echo "rc=$?" >> $O/pytest.log
