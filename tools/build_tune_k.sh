#!/bin/bash
# Rebuild only the given per-K tuning objects (e.g. 03 05 07) and relink libconv2d_tune.so (fast
# iteration on one K; `python -m paper_conf_cluster_luzw20_b200._build` rebuilds everything).
cd "$(dirname "$0")/.."
mkdir -p build/csrc_obj_tune
for k in "$@"; do
  nvcc -gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -std=c++17 -Xcompiler -fPIC --ftz=false \
    --prec-div=true --prec-sqrt=true --fmad=true -DC2D_TUNING -I include -w -c -o build/csrc_obj_tune/inst_k$k.o \
    paper_conf_cluster_luzw20_b200/csrc/inst_k$k.cu &
done
wait
nvcc -gencode arch=compute_100a,code=sm_100a -shared -cudart static -o paper_conf_cluster_luzw20_b200/libconv2d_tune.so \
  build/csrc_obj_tune/*.o
