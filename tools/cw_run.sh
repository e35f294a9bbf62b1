# GPU side of the cw1024 experiments: every build/cwvar variant on configs[1]-shaped batches, then one ncu capture.
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
: > gpurun_out/cw_r.txt
for v in ${CW_VARIANTS:-base}; do echo "== $v" >> gpurun_out/cw_r.txt; timeout 300 ./build/cwvar/$v 2000000 1000 ${CW_STEPS:-6} ${CW_DISTS:-0,1,2,3,4,5,6,7} >> gpurun_out/cw_r.txt 2>&1; done
if [ -n "$CW_NCU" ]; then
  timeout 600 ncu --set full --clock-control none --import-source on -k regex:cw1024 -c 1 -o gpurun_out/cw_$CW_NCU ./build/cwvar/$CW_NCU 300000 1000 1 ${CW_NCU_DIST:-0} > gpurun_out/cw_ncu.log 2>&1
fi
cat gpurun_out/cw_r.txt
