#!/bin/bash
mkdir -p gpurun_out
timeout 1200 compute-sanitizer --tool memcheck --target-processes all --error-exitcode 9 --print-limit 20 python tools/sanitize_cases.py p2p > gpurun_out/san_p2p_memcheck.log 2>&1
echo "exit $?" >> gpurun_out/san_p2p_memcheck.log
timeout 1200 compute-sanitizer --tool racecheck --target-processes all --error-exitcode 9 --print-limit 20 python tools/sanitize_cases.py p2p > gpurun_out/san_p2p_racecheck.log 2>&1
echo "exit $?" >> gpurun_out/san_p2p_racecheck.log
cat gpurun_out/san_p2p_*.log
