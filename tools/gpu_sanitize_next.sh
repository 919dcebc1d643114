#!/bin/bash
# compute-sanitizer memcheck / racecheck / synccheck over the SOR and Black-Scholes kernels.
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
for tool in memcheck racecheck synccheck; do
  timeout -s KILL ${SAN_TIMEOUT:-500} compute-sanitizer --tool $tool \
     python tools/sanitize_next.py > gpurun_out/r01_sanitize_next_$tool.log 2>&1
  echo "$tool rc=$?"; grep -E "ERROR SUMMARY|RACECHECK SUMMARY|Error|error" gpurun_out/r01_sanitize_next_$tool.log | tail -3
done
