#!/bin/bash
# store cache hints at mid sizes: default vs .cs (evict-first) output stores
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out /tmp/x
F="-std=c++17 -O3 -gencode arch=compute_100a,code=sm_100a -lineinfo -Ipaper_conf_asplos_phothilimthanaara13_b200/csrc"
nvcc $F tools/explore_mid.cu -o /tmp/x/em_def -lcuda &
nvcc $F '-DSEPCONV_ST_HINT=".cs"' tools/explore_mid.cu -o /tmp/x/em_cs -lcuda &
wait
for rep in 1 2; do
for b in def cs; do
  echo "== $b" ; EXPLORE_HINT=1 timeout -s KILL 600 /tmp/x/em_$b 2048 3520 4096 16384 | grep -v "^skip"
done
done > gpurun_out/r02h_hint.txt 2>&1
cat gpurun_out/r02h_hint.txt
