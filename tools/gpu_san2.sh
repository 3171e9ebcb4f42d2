#!/bin/bash
# sanitizer runs of the persistent CG kernel and the 2-process p2p transport
mkdir -p gpurun_out
timeout 300 python tools/sanitize_cases.py persist p2p > gpurun_out/san_plain.log 2>&1; echo "plain exit $?" >> gpurun_out/san_plain.log
for tool in memcheck racecheck synccheck; do
  timeout 900 compute-sanitizer --tool $tool --error-exitcode 9 --print-limit 20 python tools/sanitize_cases.py persist > gpurun_out/san_persist_$tool.log 2>&1
  echo "exit $?" >> gpurun_out/san_persist_$tool.log
done
timeout 1200 compute-sanitizer --tool memcheck --target-processes all --error-exitcode 9 --print-limit 20 python tools/sanitize_cases.py p2p > gpurun_out/san_p2p_memcheck.log 2>&1
echo "exit $?" >> gpurun_out/san_p2p_memcheck.log
tail -3 gpurun_out/san_*.log
