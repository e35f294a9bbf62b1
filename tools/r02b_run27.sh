# split kernel: 640-thread blocks (96 regs, no spill) with / without the bulk store vs 768 (default)
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
DISTS="dup16 special_mix" TAG=r02b_sp640 bash tools/ab_lib.sh > /dev/null 2>&1
cat gpurun_out/ab_r02b_sp640.txt
