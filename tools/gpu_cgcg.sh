#!/bin/bash
# NEXT-1 check: CG tests (both variants), dist/p2p, bench with the variant comparison
mkdir -p gpurun_out
timeout 1200 python -m pytest tests/test_gpu_cgcg.py tests/test_gpu_cg.py tests/test_gpu_dist.py tests/test_gpu_p2p_mp.py -x -q > gpurun_out/pytest_cg.log 2>&1
echo "pytest exit $?" >> gpurun_out/pytest_cg.log
timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu > gpurun_out/bench_tb.json 2> gpurun_out/bench_tb.err
timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu --cg-variant cgcg > gpurun_out/bench_cgcg.json 2> gpurun_out/bench_cgcg.err
tail -3 gpurun_out/pytest_cg.log
cat gpurun_out/bench_tb.json gpurun_out/bench_cgcg.json
