# loads in flight per lane (XP_U) re-swept on the final kernel
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02ak; mkdir -p $O
for v in product u8 u10 u11 product; do
  if [ $v = product ]; then L=""; else L=tools/variants/lib_$v.so; fi
  SPMV_LIB_PATH=$L timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu > $O/b.json 2> $O/b.err
  python -c "
import json; d=json.load(open('$O/b.json')); print('$v', d['value'], d['spmv']['us_avg'])" >> $O/ab.txt
done
