# cg variant 3 (fused update into the next SpMV): parity + bench
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02ai; mkdir -p $O
timeout 1500 python -m pytest tests/test_gpu_fused.py -q -x > $O/pytest.log 2>&1; echo "rc=$?" >> $O/pytest.log
timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/bench.json 2> $O/bench.err
python -c "
import json; d=json.load(open('$O/bench.json')); print(d['value'], d['cg_variants'], d['spmv']['us_avg'])" > $O/summary.txt 2>&1
