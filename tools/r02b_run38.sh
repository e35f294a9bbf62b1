cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
DISTS="dup16 special_mix" BASE_ENV="X=1" TAG=r02b_spblk3 bash tools/ab_lib.sh > /dev/null 2>&1
cat gpurun_out/ab_r02b_spblk3.txt
