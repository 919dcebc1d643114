#!/bin/bash
# A/B of the tuner's sustained confirmation (R28): previous vs current library, alternating
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
L=paper_conf_asplos_phothilimthanaara13_b200/libsepconv.so
B="timeout -s KILL 900 python bench.py --no-cpu-baseline --no-e2e --steps 20 --warmup 5"
for r in 1 2 3; do
  cp libsepconv_old.so $L; $B > gpurun_out/r02sa_old_$r.json 2>/dev/null
  cp libsepconv_new.so $L; SEPCONV_TUNE_LOG=gpurun_out/r02sa_tune_$r.log $B > gpurun_out/r02sa_new_$r.json 2>/dev/null
done
python tools/bench_summary.py gpurun_out/r02sa_*.json
grep -h sustained gpurun_out/r02sa_tune_1.log | head -30
