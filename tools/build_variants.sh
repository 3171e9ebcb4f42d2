#!/bin/bash
# Build libspmv variants with extra nvcc flags into tools/variants/ (the product
# .so is never touched):  tools/build_variants.sh NAME "FLAGS" [NAME "FLAGS" ...]
# Sweep-only knobs (-DSPMV_TUNING, XP_U_DEF, SELL_U, ...) exist only in such builds.
set -e
mkdir -p tools/variants
while [ $# -gt 0 ]; do
  name=$1; flags=$2; shift 2
  python paper_conf_asplos_ginsbachrsbdo18_b200/build.py --force --out tools/variants/lib_$name.so $flags >/dev/null \
    && echo built $name
done
