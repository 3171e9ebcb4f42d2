#!/bin/bash
# time stencil build variants (tools/variants/lib_*.so) and z-chunk sizes on 256^3
L=paper_conf_asplos_ginsbachrsbdo18_b200/libspmv_b200.so
cp $L /tmp/orig_lib.so
for v in /tmp/orig_lib.so tools/variants/lib_*.so; do
  cp $v $L
  for z in 0 26 13 8 7 4; do
    if [ $z = 0 ]; then timeout 60 python tools/time_stencil.py $(basename $v .so) 256; else timeout 60 python tools/time_stencil.py $(basename $v .so) 256 SPMV_STENCIL_ZCHUNK=$z; fi
  done
done
cp /tmp/orig_lib.so $L
