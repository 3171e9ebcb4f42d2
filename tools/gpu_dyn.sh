cd $GRAFT_REPO_ROOT
O=gpurun_out/dyn; mkdir -p $O
T() { timeout 120 python tools/time_one.py "$@" >> $O/times.jsonl 2>>$O/times.err; }
T xplan_dyn_C C xplan
T xplan_static_C C xplan SPMV_XPLAN_DYN=0
T xplan_dyn_B B xplan
T xplan_static_B B xplan SPMV_XPLAN_DYN=0
T xplan_dyn_C2 C xplan
timeout 900 python -m pytest tests/test_gpu_spmv.py -x -q -k "xplan or nas_full" > $O/pytest_spmv.log 2>&1
timeout 900 python -m pytest tests/test_gpu_cg.py tests/test_gpu_cgcg.py -x -q > $O/pytest_cg.log 2>&1
timeout 900 python -m pytest tests/test_gpu_p2p_mp.py tests/test_gpu_dist.py -x -q > $O/pytest_dist.log 2>&1
timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu > $O/bench.json 2> $O/bench.err
