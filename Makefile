# Build: libaol.so (CUDA, sm_100a, C ABI of include/aol.h) and oracle/liboracle.so (plain C, test-only).
NVCC      ?= /usr/local/cuda/bin/nvcc
PKG       := paper_conf_ipps_guortgbs11_b200
CSRC      := $(wildcard $(PKG)/csrc/*.cu)
CHDR      := $(wildcard $(PKG)/csrc/*.h $(PKG)/csrc/*.cuh) include/aol.h
LIB       := $(PKG)/libaol.so
ARCH      := -gencode arch=compute_100a,code=sm_100a
NVFLAGS   := $(ARCH) -O3 -lineinfo -std=c++17 -Xcompiler -fPIC,-fvisibility=hidden -Xptxas -v \
             --expt-relaxed-constexpr -cudart static
ORACLE    := oracle/liboracle.so

all: $(LIB) $(ORACLE)

$(LIB): $(CSRC) $(CHDR)
	$(NVCC) $(NVFLAGS) -shared -o $@.tmp $(CSRC) -lrt -ldl -lpthread 2> $(PKG)/ptxas.log || (cat $(PKG)/ptxas.log; exit 1)
	mv $@.tmp $@

$(ORACLE): oracle/aol_oracle.c oracle/aol_oracle.h
	gcc -std=c99 -O2 -fopenmp -fPIC -shared -Wall -Wextra -o $@ oracle/aol_oracle.c

clean:
	rm -f $(LIB) $(ORACLE) $(PKG)/ptxas.log

.PHONY: all clean
