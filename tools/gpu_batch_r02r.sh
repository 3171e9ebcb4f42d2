# programmatic dependent launch (PDL) of the SpMV / k_cgcg chain: parity + A/B
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02r; mkdir -p $O
timeout 1200 python -m pytest tests/test_gpu_cgcg.py tests/test_gpu_cg.py tests/test_gpu_spmv.py tests/test_gpu_persist.py tests/test_gpu_dist.py -q -x > $O/pytest.log 2>&1; echo "rc=$?" >> $O/pytest.log
for PDL in 0 1 0 1; do SPMV_PDL=$PDL timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/bench_pdl$PDL.json 2> $O/bench_pdl$PDL.err; python -c "
import json; d=json.load(open('$O/bench_pdl$PDL.json')); print('pdl=$PDL', d['value'], d['cg_variants'], d['spmv']['us_avg'], d['e2e']['value'])" >> $O/ab.txt; done
for PDL in 0 1; do SPMV_PDL=$PDL timeout 300 python tools/gap.py C rand >> $O/gap.txt 2>&1; done
