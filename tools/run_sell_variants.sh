#!/bin/bash
# SELL variants on the Parboil-shaped (sorted SELL) and stencil (SELL) matrices
L=paper_conf_asplos_ginsbachrsbdo18_b200/libspmv_b200.so
cp $L /tmp/orig_lib.so
for v in /tmp/orig_lib.so tools/variants/lib_*.so; do
  cp $v $L
  timeout 120 python tools/time_one.py $(basename $v .so) parboil auto 2>/dev/null | tail -1
  timeout 300 python tools/time_one.py $(basename $v .so) stencil256 auto 2>/dev/null | tail -1
done
cp /tmp/orig_lib.so $L
