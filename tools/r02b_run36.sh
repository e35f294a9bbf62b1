# retune of the value kernel after the round-2 changes: atomics group, CE mix, prefetch
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
DISTS="paper_uniform spectra_intensity" BASE_ENV="X=1" TAG=r02b_retune bash tools/ab_lib.sh > /dev/null 2>&1
cat gpurun_out/ab_r02b_retune.txt
