#!/bin/bash
L=paper_conf_asplos_ginsbachrsbdo18_b200/libspmv_b200.so
cp $L /tmp/orig_lib.so
for v in /tmp/orig_lib.so tools/variants/lib_*.so; do
  cp $v $L
  echo $v; timeout 120 python tools/bench_idioms.py --no-cpu jds_parboil 2>&1 | tail -1
done
cp /tmp/orig_lib.so $L
