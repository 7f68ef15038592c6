# Native build for ocelot-b200.  sm_100a only (B200); nvcc cross-compiles without a GPU.
NVCC      ?= /usr/local/cuda/bin/nvcc
CXX       ?= g++
CC        ?= gcc
ARCH      := -gencode arch=compute_100a,code=sm_100a
NVFLAGS   := $(ARCH) -O3 -lineinfo -std=c++17 -Xcompiler -fPIC -Xcompiler -Wall --expt-relaxed-constexpr -Xptxas -v
PKG       := paper_journals_pvldb_heimelspmm13_b200
LIB       := $(PKG)/_lib/libocelot_b200.so
CSRC      := $(wildcard $(PKG)/csrc/*.cu)
CHDR      := $(wildcard $(PKG)/csrc/*.cuh) include/ocelot_b200.h

all: $(LIB) oracle/liboracle.so datagen/liboclgen_host.so datagen/liboclgen_dev.so

OBJDIR    := build/obj
COBJ      := $(patsubst $(PKG)/csrc/%.cu,$(OBJDIR)/%.o,$(CSRC))

# product library: hand-written CUDA kernels + C ABI (no torch types)
$(OBJDIR)/%.o: $(PKG)/csrc/%.cu $(CHDR)
	@mkdir -p $(OBJDIR)
	$(NVCC) $(NVFLAGS) -Iinclude -c -o $@ $< 2> $(OBJDIR)/$*.ptxas.log || (cat $(OBJDIR)/$*.ptxas.log; exit 1)

# NVRTC sources of the run-time specialised kernels (jit.cu): the device headers as strings
JITHDR    := $(PKG)/csrc/spec_device.cuh $(PKG)/csrc/bulk.cuh $(PKG)/csrc/rowops.cuh $(PKG)/csrc/common.cuh include/ocelot_b200.h
$(OBJDIR)/jit_src.inc: $(JITHDR) tools/embed_src.py
	@mkdir -p $(OBJDIR)
	python3 tools/embed_src.py $@ $(JITHDR)

$(OBJDIR)/jit.o: $(PKG)/csrc/jit.cu $(CHDR) $(OBJDIR)/jit_src.inc
	@mkdir -p $(OBJDIR)
	$(NVCC) $(NVFLAGS) -Iinclude -I$(OBJDIR) -c -o $@ $< 2> $(OBJDIR)/jit.ptxas.log || (cat $(OBJDIR)/jit.ptxas.log; exit 1)

$(LIB): $(COBJ)
	@mkdir -p $(PKG)/_lib
	$(NVCC) $(ARCH) -shared -o $@ $(COBJ) -lcudart -ldl
	@cat $(OBJDIR)/*.ptxas.log > $(PKG)/_lib/ptxas.log

# oracle: test infrastructure only; plain C++17, single-threaded, no FMA contraction
oracle/liboracle.so: oracle/oracle.cpp oracle/oracle.h
	$(CXX) -O2 -std=c++17 -ffp-contract=off -fno-fast-math -fPIC -shared -o $@ oracle/oracle.cpp

# seeded input generators shared by both sides (no method arithmetic)
datagen/liboclgen_host.so: datagen/datagen_host.c datagen/ocl_datagen.h
	$(CC) -O2 -pthread -ffp-contract=off -fPIC -shared -o $@ datagen/datagen_host.c -lm

datagen/liboclgen_dev.so: datagen/datagen_dev.cu datagen/ocl_datagen.h
	$(NVCC) $(ARCH) -O3 -Xcompiler -fPIC -shared -o $@ datagen/datagen_dev.cu -lcudart

clean:
	rm -rf $(OBJDIR)
	rm -f $(LIB) oracle/liboracle.so datagen/liboclgen_host.so datagen/liboclgen_dev.so

.PHONY: all clean

# compute-sanitizer over one small call of every kernel family (tools/sanitize_cases.py checks each
# result against the oracle); needs a GPU.  Logs: profiles/sanitize_<tool>.log
SANITIZER ?= /usr/local/cuda/bin/compute-sanitizer
sanitize: all
	@for t in memcheck racecheck synccheck; do \
	  echo "== $$t"; \
	  $(SANITIZER) --tool $$t --error-exitcode 1 --print-limit 20 python tools/sanitize_cases.py $(CASES) \
	    > profiles/sanitize_$$t.log 2>&1; echo "rc=$$?"; tail -3 profiles/sanitize_$$t.log; \
	done

.PHONY: sanitize
