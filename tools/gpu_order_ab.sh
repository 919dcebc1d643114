#!/bin/bash
# does the order of the widths inside a step matter under the power cap?  A/B, interleaved runs
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
B="timeout -s KILL 900 python bench.py --steps 20 --warmup 5 --no-cpu-baseline --no-e2e"
for r in 1 2; do
  $B > gpurun_out/r02n_order_asc_$r.json 2>/dev/null
  $B --widths 3,17,5,15,7,13,9,11 > gpurun_out/r02n_order_mix_$r.json 2>/dev/null
done
python tools/bench_summary.py gpurun_out/r02n_order_*.json
