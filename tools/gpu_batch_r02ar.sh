# JDS: two units per warp in lockstep (batch 2/4/8) vs one
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02ar; mkdir -p $O
SPMV_LIB_PATH=tools/variants/lib_jdspair.so timeout 900 python -m pytest tests/test_gpu_jds.py -q -x > $O/pytest.log 2>&1; echo "rc=$?" >> $O/pytest.log
for v in product jdspair jdspair8 jdspair2 product; do
  if [ $v = product ]; then L=""; else L=tools/variants/lib_$v.so; fi
  echo "== $v" >> $O/jds.jsonl
  SPMV_LIB_PATH=$L timeout 300 python tools/bench_idioms.py jds_parboil >> $O/jds.jsonl 2>> $O/jds.err
done
