# the update kernel: PDL on/off (placement on the SpMV's idle SMs vs all SMs) and grid size
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02aj; mkdir -p $O
export SPMV_LIB_PATH=tools/variants/lib_tuning.so
for cfg in "SPMV_PDL_UPD=1" "SPMV_PDL_UPD=0" "SPMV_UPD_GRID=56" "SPMV_UPD_GRID=28" "SPMV_UPD_GRID=296 SPMV_PDL_UPD=0" "SPMV_PDL_UPD=1"; do
  env $cfg timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu --cg-variant cgcg > $O/b.json 2> $O/b.err
  python -c "
import json; d=json.load(open('$O/b.json')); print('$cfg', d['value'], d['cg_variants'].get('textbook'), d['spmv']['us_avg'])" >> $O/ab.txt
done
