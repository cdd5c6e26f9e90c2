# Build of every native artefact, in-tree (the .so files travel to the GPU
# box with the gpurun snapshot).  `make -j` from the repo root.
NVCC    ?= /usr/local/cuda/bin/nvcc
CXX     ?= g++
ARCH    := -gencode arch=compute_100a,code=sm_100a
NVFLAGS := $(ARCH) -O3 -lineinfo -std=c++17 -Xcompiler -fPIC -Xcompiler -Wall --expt-relaxed-constexpr
CXXFLAGS:= -O2 -std=c++17 -fPIC -Wall -Wextra

PKG     := paper_journals_pvldb_pirkmzm16_b200
CSRC    := $(PKG)/csrc
LIBVD   := $(PKG)/libvd.so
LIBGEN  := gen/libvdgen.so
LIBOR   := oracle/liboracle.so

VD_CU   := $(wildcard $(CSRC)/*.cu)
VD_CPP  := $(wildcard $(CSRC)/*.cpp)
VD_HDR  := $(wildcard $(CSRC)/*.cuh) $(wildcard $(CSRC)/*.h) include/vd.h
VD_OBJ  := $(patsubst %.cu,build/%.o,$(VD_CU)) $(patsubst %.cpp,build/%.o,$(VD_CPP))

all: $(LIBOR) $(LIBGEN) $(LIBVD)

# --- oracle: plain C++17, single-threaded, no CUDA ----------------------
$(LIBOR): oracle/voodoo_oracle.cpp oracle/tpch_oracle.cpp oracle/oracle.h
	$(CXX) $(CXXFLAGS) -shared -o $@ oracle/voodoo_oracle.cpp oracle/tpch_oracle.cpp

# --- shared input generator (host + device fill) -------------------------
$(LIBGEN): gen/vdgen.cu gen/vd_gen.h
	$(NVCC) $(NVFLAGS) -shared -o $@ gen/vdgen.cu

# --- product library -------------------------------------------------------
build/$(CSRC)/%.o: $(CSRC)/%.cu $(VD_HDR)
	@mkdir -p $(dir $@)
	$(NVCC) $(NVFLAGS) -Iinclude -I$(CSRC) -Xptxas -v -c -o $@ $< 2> $@.ptxas.txt || (cat $@.ptxas.txt; false)

build/$(CSRC)/%.o: $(CSRC)/%.cpp $(VD_HDR)
	@mkdir -p $(dir $@)
	$(CXX) $(CXXFLAGS) -I/usr/local/cuda/include -Iinclude -I$(CSRC) -c -o $@ $<

$(LIBVD): $(VD_OBJ)
	$(NVCC) $(ARCH) -shared -o $@ $(VD_OBJ) -lcudart

clean:
	rm -rf build $(LIBVD) $(LIBGEN) $(LIBOR)

.PHONY: all clean
