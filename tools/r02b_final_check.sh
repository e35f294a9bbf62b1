# final check of the last build: smoke, full GPU suite, headline bench line
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/f_smoke.log 2>&1; echo smoke rc=$? >> gpurun_out/f_smoke.log
timeout 1800 python -m pytest tests -q -m gpu > gpurun_out/f_pytest.log 2>&1; echo pytest rc=$? >> gpurun_out/f_pytest.log
timeout 600 python bench.py > gpurun_out/f_bench.json 2> gpurun_out/f_bench.err
tail -2 gpurun_out/f_smoke.log; tail -3 gpurun_out/f_pytest.log; tail -1 gpurun_out/f_bench.json | cut -c1-400
