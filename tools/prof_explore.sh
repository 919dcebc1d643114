cd $GRAFT_REPO_ROOT
for K in 11 13; do
ncu --set full --clock-control none -k regex:stream_kernel -s 1 -c 1 -o gpurun_out/r01_exp_k$K ./tools/explore 1 $K > gpurun_out/r01_exp_k$K.log 2>&1
done
ls -la gpurun_out/
