# persisting-L2 window over the CG vectors (one workspace): parity + A/B
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02ae; mkdir -p $O
timeout 1500 python -m pytest tests/test_gpu_cg.py tests/test_gpu_cgcg.py tests/test_gpu_persist.py tests/test_gpu_dist.py tests/test_gpu_p2p_mp.py tests/test_gpu_launch_modes.py -q -x > $O/pytest.log 2>&1; echo "rc=$?" >> $O/pytest.log
SPMV_CG_L2WIN=1 timeout 1500 python -m pytest tests/test_gpu_cg.py tests/test_gpu_cgcg.py -q -x > $O/pytest_win.log 2>&1; echo "rc=$?" >> $O/pytest_win.log
for W in 0 1 0 1; do SPMV_CG_L2WIN=$W timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/bench_w$W.json 2> $O/bench_w$W.err; python -c "
import json; d=json.load(open('$O/bench_w$W.json')); print('win=$W', d['value'], d['cg_variants'], d['spmv']['us_avg'], d['e2e']['value'])" >> $O/ab.txt; done
