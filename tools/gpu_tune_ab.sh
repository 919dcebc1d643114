#!/bin/bash
# tuner with fewer-CTA seeds and a wider mutation pool: bench A/B (default run) and the mid sizes
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
B="timeout -s KILL 900 python bench.py --no-cpu-baseline --no-e2e"
( time $B --steps 20 --warmup 5 > gpurun_out/r02q_bench_c4_a.json 2> gpurun_out/r02q_bench_c4_a.err ) 2> gpurun_out/r02q_time.txt
$B --steps 20 --warmup 5 > gpurun_out/r02q_bench_c4_b.json 2> /dev/null
$B --steps 50 --warmup 3 --size 2048 --widths 3,7,11,15,17 > gpurun_out/r02q_bench_c2.json 2>/dev/null
$B --steps 50 --warmup 3 --size 4096 --widths 17 > gpurun_out/r02q_bench_c3.json 2>/dev/null
$B --steps 50 --warmup 3 --size 3520 > gpurun_out/r02q_bench_c2p.json 2>/dev/null
$B --steps 5 --warmup 3 --workload batch > gpurun_out/r02q_bench_c5.json 2>/dev/null
python tools/bench_summary.py gpurun_out/r02q_bench_*.json
cat gpurun_out/r02q_time.txt
