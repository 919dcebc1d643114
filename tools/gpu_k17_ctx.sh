#!/bin/bash
# K=17 inside the bench step vs alone vs after K=15 only: where do the 5-9% go?
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
B="timeout -s KILL 900 python bench.py --no-cpu-baseline --no-e2e --steps 20 --warmup 5"
$B --widths 17 > gpurun_out/r02t_k17_alone.json 2>/dev/null
$B --widths 15,17 > gpurun_out/r02t_k15_17.json 2>/dev/null
$B --widths 3,17 > gpurun_out/r02t_k3_17.json 2>/dev/null
$B > gpurun_out/r02t_all.json 2>/dev/null
$B --widths 17 > gpurun_out/r02t_k17_alone_b.json 2>/dev/null
python tools/bench_summary.py gpurun_out/r02t_*.json
for f in gpurun_out/r02t_*.json; do python -c "
import json,sys; d=json.loads(open('$f').read().strip().splitlines()[-1]); print('$f', d['clocks'], {k: round(v['tuned_us'],1) for k,v in d['per_width'].items()})"; done
