#!/bin/bash
# mid-size benches after the right-edge change (BASELINE C2, C3, the paper's 3520^2), --steps 100
mkdir -p gpurun_out
for spec in "2048 3,7,11,15,17 c2" "4096 17 c3" "3520 3,5,7,9,11,13,15,17 c2p"; do
  set -- $spec
  timeout -s KILL 600 python bench.py --size $1 --widths $2 --steps 100 --no-cpu-baseline > gpurun_out/bench_$3_s100.json 2> gpurun_out/bench_$3.err
  python tools/bench_summary.py gpurun_out/bench_$3_s100.json
done
timeout -s KILL 300 python tools/copy_floor.py --sizes 2048,3520,4096 --widths 3,9,17 | tee gpurun_out/copy_floor_after.txt
