#!/bin/bash
# per-instruction shared-memory bank conflicts of the fused kernel (ncu SourceCounters, SASS page)
cd "${GRAFT_REPO_ROOT:-$(dirname "$0")/..}"
mkdir -p gpurun_out
for spec in 3:sep-fused-tma2 9:sep-fused-tma0 17:sep-fused-tma4; do
  K=${spec%%:*}; C=${spec#*:}
  timeout -s KILL 600 ncu --section SourceCounters --section MemoryWorkloadAnalysis_Tables --import-source on --clock-control none \
     -k regex:stream_kernel -s 1 -c 1 -o /tmp/bank_k$K python tools/prof_one.py --k $K --cand $C --n 1 --size 4096 > gpurun_out/r02k_bank_k$K.log 2>&1
  echo "K=$K rc=$?"
  ncu -i /tmp/bank_k$K.ncu-rep --page source --csv --print-source sass > gpurun_out/r02k_bank_src_k$K.csv 2>>gpurun_out/r02k_bank_k$K.log
  ncu -i /tmp/bank_k$K.ncu-rep --page raw --csv > gpurun_out/r02k_bank_raw_k$K.csv 2>>gpurun_out/r02k_bank_k$K.log
done
ls -la gpurun_out/
