# elect.sync single-lane bulk ops (GAS_BK_ELECT) A/B + its parity
cd $GRAFT_REPO_ROOT
mkdir -p gpurun_out
GAS_LIB=$PWD/build/variants/libgas_elect.so timeout 900 python -m pytest tests/test_gpu_keylin.py tests/test_gpu_bucket.py -x -q -k "not cta and not offsets" > gpurun_out/pytest_el.log 2>&1; echo pytest rc=$? >> gpurun_out/pytest_el.log
DISTS="paper_uniform spectra_intensity uniform_bits" BASE_ENV="X=1" TAG=r02b_el bash tools/ab_lib.sh > /dev/null 2>&1
tail -3 gpurun_out/pytest_el.log; cat gpurun_out/ab_r02b_el.txt
