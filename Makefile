# Builds the product library (CUDA sm_100a + C++ host engine) in-tree.
# The oracle (oracle/) and the input generator (swgen/) are built by their own
# Python build() helpers (plain gcc); __graft_entry__.build() runs all three.
NVCC    ?= nvcc
ARCH    := -gencode arch=compute_100a,code=sm_100a
PKG     := paper_conf_icpp_kedad_sidhoummmmt14_b200
SRC     := $(PKG)/csrc
OBJ     := build/obj
LIB     := $(PKG)/libswdual.so
NVFLAGS := $(ARCH) -O3 -lineinfo -std=c++17 -Xcompiler -fPIC,-Wall -Iinclude
HDRS    := include/swdual.h $(wildcard $(SRC)/*.h $(SRC)/*.cuh)
OBJS    := $(OBJ)/kernels.o $(OBJ)/align.o $(OBJ)/cpu_striped.o $(OBJ)/engine.o $(OBJ)/packer.o $(OBJ)/sched.o

all: $(LIB)

$(OBJ)/%.o: $(SRC)/%.cu $(HDRS)
	@mkdir -p $(OBJ)
	$(NVCC) $(NVFLAGS) -c $< -o $@

# CPU-type PE kernel (hybrid SWDUAL): AVX2 in this file only; sw_search_cpu checks the CPU first
$(OBJ)/cpu_striped.o: $(SRC)/cpu_striped.cpp $(HDRS)
	@mkdir -p $(OBJ)
	$(NVCC) $(NVFLAGS) -Xcompiler -mavx2 -c $< -o $@

$(OBJ)/%.o: $(SRC)/%.cpp $(HDRS)
	@mkdir -p $(OBJ)
	$(NVCC) $(NVFLAGS) -c $< -o $@

$(LIB): $(OBJS)
	$(NVCC) $(ARCH) -shared -Xlinker --no-undefined -o $@.tmp $(OBJS) -lcudart_static -lrt -lpthread -ldl && mv $@.tmp $@

clean:
	rm -rf build $(LIB)

.PHONY: all clean
