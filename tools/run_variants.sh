#!/bin/bash
# run_variants.sh MATRIX KERNEL [ENV...]: time every tools/variants/lib_*.so (swapped in)
L=paper_conf_asplos_ginsbachrsbdo18_b200/libspmv_b200.so
cp $L /tmp/orig_lib.so
for v in tools/variants/lib_*.so; do
  cp $v $L
  timeout 60 python tools/time_one.py $(basename $v .so) "$@" 2>&1 | tail -1
done
cp /tmp/orig_lib.so $L
