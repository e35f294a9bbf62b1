# merged overflow vote: offsets + CTA parity; counting-sort CE mix A/B on spectra_intensity; configs[3] bench
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 1200 python -m pytest tests/test_gpu_parity.py tests/test_gpu_bucket.py tests/test_gpu_cluster.py -x -q > gpurun_out/pytest_cta.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_cta.log
DISTS="spectra_intensity" BASE_ENV="X=1" TAG=r02b_cwmix bash tools/ab_lib.sh > /dev/null 2>&1
timeout 300 python bench.py --config 3 --steps 10 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/c3_merge.log 2>&1
tail -3 gpurun_out/pytest_cta.log; cat gpurun_out/ab_r02b_cwmix.txt; tail -1 gpurun_out/c3_merge.log | cut -c1-300
