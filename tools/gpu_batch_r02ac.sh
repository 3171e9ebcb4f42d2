# JDS: diagonal offsets preloaded per unit (no jds_ptr round trip per batch), batch 4/8/16, vs the previous kernel
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02ac; mkdir -p $O
timeout 900 python -m pytest tests/test_gpu_jds.py -q -x > $O/pytest.log 2>&1; echo "rc=$?" >> $O/pytest.log
for v in product jdsold jdsb4 jdsb16; do
  if [ $v = product ]; then L=""; else L=tools/variants/lib_$v.so; fi
  echo "== $v" >> $O/jds.jsonl
  SPMV_LIB_PATH=$L timeout 300 python tools/bench_idioms.py jds_parboil >> $O/jds.jsonl 2>> $O/jds.err
done
