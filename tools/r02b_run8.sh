# cluster path (f4) rework: parity + sweep; sampler trim: dists + launch list
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_cluster.py tests/test_gpu_keylin.py -x -q > gpurun_out/pytest_cl.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_cl.log
SKIP_TESTS=1 SWEEP="16385:122000 20000:100000 24576:81000 24577:81000 32768:61000 40000:50000 49152:40000 65536:30500" bash tools/sweep.sh > /dev/null 2>&1
DISTS="paper_uniform spectra_intensity" TAG=r02b_s3 bash tools/dists_run.sh > /dev/null 2>&1
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/r02b_launches_uniform2.csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline > /dev/null 2>&1
tail -3 gpurun_out/pytest_cl.log; cat gpurun_out/sweep.log gpurun_out/dists_r02b_s3.txt
