#!/bin/bash
# build libspmv variants with -D flags: build_variants.sh NAME "FLAGS" [NAME "FLAGS" ...]
ND=$(python -c "import paper_conf_asplos_ginsbachrsbdo18_b200.build as b; print(b.nccl_dir())" 2>/dev/null || echo /opt/prime-rl/.venv/lib/python3.12/site-packages/nvidia/nccl)
mkdir -p tools/variants
while [ $# -gt 0 ]; do
  name=$1; flags=$2; shift 2
  nvcc -gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -std=c++17 -Xcompiler -fPIC -shared $flags \
    -I include -I $ND/include paper_conf_asplos_ginsbachrsbdo18_b200/csrc/spmv_abi.cu -o tools/variants/lib_$name.so \
    -L $ND/lib -l:libnccl.so.2 -Xlinker=-rpath=$ND/lib -cudart static && echo built $name
done
