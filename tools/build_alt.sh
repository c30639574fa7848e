#!/bin/bash
# build an alternative libconv2d (extra -D flags) for A/B timing: tools/build_alt.sh NAME "-DFLAG=..."
# -> paper_conf_cluster_luzw20_b200/libconv2d_NAME.so (use with C2D_LIB=<that path>)
cd "$(dirname "$0")/.."
NAME=$1; shift
OUT=build/alt_$NAME; mkdir -p $OUT
for f in paper_conf_cluster_luzw20_b200/csrc/*.cu; do
  /usr/local/cuda/bin/nvcc -gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -std=c++17 -Xcompiler -fPIC \
    --ftz=false --prec-div=true --prec-sqrt=true --fmad=true -I include "$@" -c -o $OUT/$(basename $f .cu).o $f 2>/dev/null &
done
wait
/usr/local/cuda/bin/nvcc -gencode arch=compute_100a,code=sm_100a -shared -cudart static -o paper_conf_cluster_luzw20_b200/libconv2d_$NAME.so $OUT/*.o
ls -la paper_conf_cluster_luzw20_b200/libconv2d_$NAME.so
