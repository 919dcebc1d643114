#!/bin/bash
# A/B of the 8-byte right-edge store change: the same harness compiled against the previous and
# the current kernels header, interleaved on one box.  The previous header is not kept in the tree;
# recreate it before running:
#   mkdir -p tools/ab_old && git show 0423900:paper_conf_asplos_phothilimthanaara13_b200/csrc/sepconv_kernels.cuh \
#       > tools/ab_old/sepconv_kernels.cuh && cp paper_conf_asplos_phothilimthanaara13_b200/csrc/sepconv_params.h tools/ab_old/
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out /tmp/x
F="-std=c++17 -O3 -gencode arch=compute_100a,code=sm_100a"
nvcc $F -Itools/ab_old -Ipaper_conf_asplos_phothilimthanaara13_b200/csrc tools/explore_mid.cu -o /tmp/x/em_old -lcuda &
nvcc $F -Ipaper_conf_asplos_phothilimthanaara13_b200/csrc tools/explore_mid.cu -o /tmp/x/em_new -lcuda &
wait
for r in 1 2 3; do
  echo "== old"; EXPLORE_EDGE8=1 timeout -s KILL 600 /tmp/x/em_old 16384 2048 3520 | grep -v skip
  echo "== new"; EXPLORE_EDGE8=1 timeout -s KILL 600 /tmp/x/em_new 16384 2048 3520 | grep -v skip
done > gpurun_out/r02x_edge8_ab.txt 2>&1
cat gpurun_out/r02x_edge8_ab.txt
