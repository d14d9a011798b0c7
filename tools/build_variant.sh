#!/bin/bash
# Build an A/B variant of libswdual.so with extra -D flags for kernels.cu and engine.cpp:
#   bash tools/build_variant.sh NAME -DSW_X=0 ...   -> build/variants/NAME.so
set -e
name=$1; shift
mkdir -p build/variants/$name.obj
nvcc -gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -std=c++17 -Xcompiler -fPIC,-Wall -Iinclude "$@" \
  -c paper_conf_icpp_kedad_sidhoummmmt14_b200/csrc/kernels.cu -o build/variants/$name.obj/kernels.o
nvcc -gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -std=c++17 -Xcompiler -fPIC,-Wall -Iinclude "$@" \
  -c paper_conf_icpp_kedad_sidhoummmmt14_b200/csrc/engine.cpp -o build/variants/$name.obj/engine.o
nvcc -gencode arch=compute_100a,code=sm_100a -shared -Xlinker --no-undefined -o build/variants/$name.so \
  build/variants/$name.obj/kernels.o build/obj/align.o build/obj/cpu_striped.o build/variants/$name.obj/engine.o build/obj/packer.o \
  build/obj/sched.o -lcudart_static -lrt -lpthread -ldl
