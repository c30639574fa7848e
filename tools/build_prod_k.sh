#!/bin/bash
# Rebuild only the given per-K product objects (e.g. 09 11 13) and relink libconv2d.so (fast iteration).
cd "$(dirname "$0")/.."
for k in "$@"; do
  nvcc -gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -std=c++17 -Xcompiler -fPIC --ftz=false \
    --prec-div=true --prec-sqrt=true --fmad=true -I include -w -c -o build/csrc_obj/inst_k$k.o \
    paper_conf_cluster_luzw20_b200/csrc/inst_k$k.cu &
done
wait
nvcc -gencode arch=compute_100a,code=sm_100a -shared -cudart static -o paper_conf_cluster_luzw20_b200/libconv2d.so \
  build/csrc_obj/*.o
