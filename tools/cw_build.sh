# Build the cw1024 experiment variants: tools/cw_build.sh name [-Dflags...] (run from the repo root)
set -e
name=$1; shift
mkdir -p build/cwvar
nvcc -gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -std=c++17 "$@" -Xcompiler -fPIC,-fvisibility=hidden -shared -o build/cwvar/libcw_$name.so tools/cw_lib.cu
nvcc -gencode arch=compute_100a,code=sm_100a -O3 -std=c++17 -I include -I datagen -o build/cwvar/$name tools/cw_exp.cu \
  -L build/cwvar -l:libcw_$name.so -L paper_conf_icppw_awans16_b200 -l:libgas.so -L datagen -l:libgasgen.so \
  -Xlinker -rpath,'$ORIGIN' -Xlinker -rpath,'$ORIGIN/../../paper_conf_icppw_awans16_b200' -Xlinker -rpath,'$ORIGIN/../../datagen'
