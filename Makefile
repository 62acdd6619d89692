# Build: libaol.so (CUDA, sm_100a, C ABI of include/aol.h) and oracle/liboracle.so (plain C, test-only).
# Objects compile in parallel (`make -j`); ptxas register/spill reports land in build/*.ptxas.log.
NVCC      ?= /usr/local/cuda/bin/nvcc
PKG       := paper_conf_ipps_guortgbs11_b200
CSRC      := $(wildcard $(PKG)/csrc/*.cu)
CHDR      := $(wildcard $(PKG)/csrc/*.h $(PKG)/csrc/*.cuh) include/aol.h
BUILD     ?= build
OBJS      := $(patsubst $(PKG)/csrc/%.cu,$(BUILD)/%.o,$(CSRC))
LIB       ?= $(PKG)/libaol.so
ARCH      := -gencode arch=compute_100a,code=sm_100a
NVFLAGS   := $(ARCH) -O3 -lineinfo -std=c++17 -Xcompiler -fPIC,-fvisibility=hidden -Xptxas -v \
             --expt-relaxed-constexpr -I $(BUILD) $(EXTRA)
ORACLE    := oracle/liboracle.so
SYNTH     := synth/libsynth.so

EXAMPLE   := $(BUILD)/aol_example

all: $(LIB) $(ORACLE) $(SYNTH) $(EXAMPLE)

$(BUILD)/%.o: $(PKG)/csrc/%.cu $(CHDR)
	@mkdir -p $(BUILD)
	$(NVCC) $(NVFLAGS) -c -o $@ $< 2> $(BUILD)/$*.ptxas.log || (cat $(BUILD)/$*.ptxas.log; exit 1)

# the separable chain kernel's body as a string literal, compiled again at run time by NVRTC (chain_sep.cu)
$(BUILD)/sep_body.inc: $(PKG)/csrc/sep_body.cuh
	@mkdir -p $(BUILD)
	{ printf 'R"AOLSEPBODY('; cat $<; printf ')AOLSEPBODY"\n'; } > $@

$(BUILD)/chain_sep.o: $(BUILD)/sep_body.inc

$(LIB): $(OBJS)
	$(NVCC) $(ARCH) -shared -cudart static -o $@.tmp $(OBJS) -lrt -ldl -lpthread
	mv $@.tmp $@

# a plain-C client of the C ABI (no Python): examples/aol_example.c
$(EXAMPLE): examples/aol_example.c include/aol.h $(LIB)
	@mkdir -p $(BUILD)
	gcc -std=c11 -O2 -Wall -Wextra -I include -I /usr/local/cuda/include $< -L $(PKG) -laol \
	    -L /usr/local/cuda/lib64 -lcudart -Wl,-rpath,'$$ORIGIN/../$(PKG)' -o $@

$(ORACLE): oracle/aol_oracle.c oracle/aol_oracle.h
	gcc -std=c99 -O2 -fopenmp -fPIC -shared -Wall -Wextra -o $@ oracle/aol_oracle.c

# the seeded input generator in C (synth/synth.c; no method arithmetic): bench-size oracle inputs
$(SYNTH): synth/synth.c
	gcc -std=c99 -O2 -fopenmp -fPIC -shared -Wall -Wextra -o $@ synth/synth.c

clean:
	rm -rf $(BUILD) $(LIB) $(ORACLE) $(SYNTH)

.PHONY: all clean
