# NAS outer iteration: x_new before the residual, its host copy overlapping the residual
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02ap; mkdir -p $O
timeout 1500 python -m pytest tests/test_gpu_cg.py tests/test_gpu_cgcg.py tests/test_gpu_persist.py tests/test_gpu_dist.py tests/test_gpu_p2p_mp.py tests/test_gpu_launch_modes.py tests/test_bench_contract.py -q -x > $O/pytest.log 2>&1; echo "rc=$?" >> $O/pytest.log
for i in 1 2; do timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/b$i.json 2> $O/b$i.err; python -c "
import json; d=json.load(open('$O/b$i.json')); print(d['value'], d['e2e']['value'], d['cg_variants'])" >> $O/ab.txt; done
