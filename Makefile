# Native build of the libraries without Python (same flags as paper_conf_icppw_awans16_b200/build.py).
#   make            libgas.so (C ABI, sm_100a), datagen/libgasgen.so, oracle/liboracle.so, tools/gas_bench
#   ./tools/gas_bench [N] [n]     C-only benchmark of gas_sort_arrays (CUDA events)
NVCC ?= nvcc
ARCH := -gencode arch=compute_100a,code=sm_100a
NVFLAGS := $(ARCH) -O3 -lineinfo -std=c++17 -Xcompiler -fPIC
PKG := paper_conf_icppw_awans16_b200
CSRC := $(wildcard $(PKG)/csrc/*.cu $(PKG)/csrc/*.cuh) include/gas.h

all: $(PKG)/libgas.so datagen/libgasgen.so oracle/liboracle.so tools/gas_bench

$(PKG)/libgas.so: $(CSRC)
	$(NVCC) $(NVFLAGS) -Xcompiler -fvisibility=hidden -shared -Xptxas -warn-spills -I include -o $@ $(wildcard $(PKG)/csrc/*.cu)

datagen/libgasgen.so: datagen/gasgen.cu datagen/gasgen.h
	$(NVCC) $(ARCH) -O3 -lineinfo -Xcompiler -fPIC -shared -o $@ datagen/gasgen.cu

oracle/liboracle.so: oracle/gas_oracle.c
	gcc -O2 -fno-fast-math -std=c11 -Wall -Wextra -shared -fPIC -o $@ $<

tools/gas_bench: tools/gas_bench.cu $(PKG)/libgas.so datagen/libgasgen.so
	$(NVCC) $(ARCH) -O3 -std=c++17 -I include -I datagen -o $@ tools/gas_bench.cu \
	  -L $(PKG) -l:libgas.so -L datagen -l:libgasgen.so -Xlinker -rpath,'$$ORIGIN/../$(PKG)' -Xlinker -rpath,'$$ORIGIN/../datagen'

clean:
	rm -f $(PKG)/libgas.so datagen/libgasgen.so oracle/liboracle.so tools/gas_bench

.PHONY: all clean
