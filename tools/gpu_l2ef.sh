#!/bin/bash
# plan streaming with an L2 evict-first policy (XP_L2EF) vs the default: CG it/s and the SpMV alone
O=gpurun_out/l2ef; mkdir -p $O; : > $O/res.txt
for rep in 1 2; do
for v in base l2ef; do
  if [ $v = base ]; then L=paper_conf_asplos_ginsbachrsbdo18_b200/libspmv_b200.so; else L=tools/variants/lib_$v.so; fi
  SPMV_LIB_PATH=$L timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu > $O/bench_$v.json 2> $O/bench_$v.err
  python -c "
import json; d=json.loads(open('$O/bench_$v.json').read().strip().splitlines()[-1])
print('$v', d['value'], d['cg_variants'], d['spmv']['us_avg'], d['spmv']['us_eager_avg'], d['e2e']['value'])" >> $O/res.txt
  echo -n "$v " >> $O/res.txt; SPMV_LIB_PATH=$L timeout 120 python tools/gap.py C rand >> $O/res.txt 2>&1
done; done
SPMV_LIB_PATH=tools/variants/lib_l2ef.so timeout 600 python -m pytest tests/test_gpu_cgcg.py tests/test_gpu_persist.py -q -x 2>&1 | tail -2 >> $O/res.txt
cat $O/res.txt
