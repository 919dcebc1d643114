#!/bin/bash
# Right-edge warps on the 16-byte store path: parity, the per-strip CTA durations, and the
# 16384^2 bench widths (profiles/r02_cta_strips.txt)
mkdir -p gpurun_out
timeout -s KILL 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fuzz.py tests/test_gpu_fullsize.py -x -q 2>&1 | tail -2
(cd tools && CTA_TRACE_STRIPS=1 timeout -s KILL 120 ./cta_trace strips) 2>&1 | grep -v "slowest\|fastest" | tee gpurun_out/cta_strips_after.txt
timeout -s KILL 300 python tools/sched_check.py --size 16384 --k 17 --cands tma4,tma2,tma3 --scheds 0:0,9:0,18:0
timeout -s KILL 300 python tools/sched_check.py --size 16384 --k 15 --cands tma2,tma4 --scheds 0:0,9:0
timeout -s KILL 900 python bench.py --no-cpu-baseline > gpurun_out/bench_strips.json 2> gpurun_out/bench_strips.err
python tools/bench_summary.py gpurun_out/bench_strips.json
python -c "
import json; d=json.load(open('gpurun_out/bench_strips.json'))
for k,v in d['per_width'].items(): print(k, v['variant'], round(v['tuned_us'],1), round(v['us'],1))
print(d['roofline']['frac'], d['clocks'])"
