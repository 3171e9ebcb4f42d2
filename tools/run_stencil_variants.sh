#!/bin/bash
# time stencil build variants (tools/variants/lib_*.so) against the in-tree library on 256^3
L=paper_conf_asplos_ginsbachrsbdo18_b200/libspmv_b200.so
cp $L /tmp/orig_lib.so
for v in /tmp/orig_lib.so tools/variants/lib_*.so; do
  cp $v $L
  for i in 1 2; do timeout 60 python tools/time_stencil.py $(basename $v .so) 256; done
done
cp /tmp/orig_lib.so $L
