# Build the sm_100a CUDA library (libhj.so, in-tree) and the CPU oracle (test infrastructure).
NVCC ?= nvcc
PKG := paper_conf_icde_sioulasckaa19_b200
NVFLAGS := -gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -std=c++17 -Xcompiler -fPIC -shared \
           -Xptxas -v --expt-relaxed-constexpr
SRCS := $(wildcard $(PKG)/csrc/*.cu $(PKG)/csrc/*.cuh) include/hj.h

all: $(PKG)/libhj.so oracle/liboracle.so

$(PKG)/libhj.so: $(SRCS)
	$(NVCC) $(NVFLAGS) -o $@ $(PKG)/csrc/hj_api.cu 2> build_ptxas.log || (cat build_ptxas.log; false)

oracle/liboracle.so: oracle/hj_oracle.c
	gcc -O2 -std=c11 -shared -fPIC -o $@ $<

clean:
	rm -f $(PKG)/libhj.so oracle/liboracle.so build_ptxas.log

.PHONY: all clean
