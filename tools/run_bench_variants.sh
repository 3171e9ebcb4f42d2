#!/bin/bash
# CG bench (class C, CG it/s) for each build variant in tools/variants
L=paper_conf_asplos_ginsbachrsbdo18_b200/libspmv_b200.so
cp $L /tmp/orig_lib.so
for v in /tmp/orig_lib.so tools/variants/lib_*.so; do
  cp $v $L
  for i in 1 2; do
    timeout 300 python bench.py --steps 10 --warmup 3 --no-cpu 2>/dev/null | python -c "import json,sys; d=json.loads(sys.stdin.read()); print('$(basename $v .so)', d['value'], d['spmv']['us_median'])"
  done
done
cp /tmp/orig_lib.so $L
