#!/bin/bash
# compute-sanitizer memcheck / racecheck / synccheck over every candidate on small shapes.
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
for tool in memcheck racecheck synccheck; do
  timeout -s KILL ${SAN_TIMEOUT:-500} compute-sanitizer --tool $tool \
     python tools/sanitize.py ${SANITIZE_KS:-3,17} > gpurun_out/${ROUND:-r02}_sanitize_$tool.log 2>&1
  echo "$tool rc=$?"; grep -E "ERROR SUMMARY|RACECHECK SUMMARY|Error|error" gpurun_out/${ROUND:-r02}_sanitize_$tool.log | tail -3
done
