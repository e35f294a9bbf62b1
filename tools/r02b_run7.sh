# sampler with the CDF phase only when needed: tests + distributions + launch list on paper_uniform
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_keylin.py tests/test_gpu_sort1024.py tests/test_gpu_split.py -x -q > gpurun_out/pytest_cdf.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_cdf.log
TAG=r02b_cdf2 bash tools/dists_run.sh > /dev/null 2>&1
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/r02b_launches_uniform.csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline > /dev/null 2>&1
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/r02b_launches_spectra.csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline --dist spectra_intensity > /dev/null 2>&1
tail -3 gpurun_out/pytest_cdf.log; cat gpurun_out/dists_r02b_cdf2.txt
