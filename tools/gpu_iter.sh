#!/bin/bash
# one GPU iteration: variant timings (C, B), GPU tests (PYTEST_ARGS), sweep (SWEEP)
mkdir -p gpurun_out
if ls tools/variants/lib_*.so >/dev/null 2>&1; then
  for m in ${VMATS:-C B}; do bash tools/run_variants.sh $m ${VKERN:-xplan}; done > gpurun_out/variants.txt 2>&1
fi
timeout 1500 python -m pytest tests -m gpu -x -q ${PYTEST_ARGS} > gpurun_out/pytest_gpu.log 2>&1; echo "pytest exit $?" >> gpurun_out/pytest_gpu.log
tail -5 gpurun_out/pytest_gpu.log
if [ -n "$SWEEP" ]; then timeout 900 python tools/sweep.py $SWEEP > gpurun_out/sweep.jsonl 2> gpurun_out/sweep.err; fi
if [ -n "$BENCH" ]; then timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu > gpurun_out/bench.json 2> gpurun_out/bench.err; cat gpurun_out/bench.json; fi
cat gpurun_out/variants.txt 2>/dev/null
