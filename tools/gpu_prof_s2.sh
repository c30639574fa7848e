#!/bin/bash
# Session-2 study batch: small-image per-call overhead by variant, ncu full captures of the weak sweep
# points (4096^2 K=15, 8192^2 K=7, 1024^2 K=3) and of the tensor-core variant on configs[2].
cd "$(dirname "$0")/.."
mkdir -p gpurun_out
timeout 300 python tools/small_sizes.py 0,1,2,3,4 > gpurun_out/small_sizes.txt 2>&1
for spec in "15 0 4096" "7 0 8192" "7 0 4096" "3 0 1024"; do timeout 300 bash tools/prof2.sh "$spec" > /dev/null 2>&1; done
n=prof_tc_config2
timeout 300 ncu --set full --clock-control none --import-source on -k regex:k_conv2d_multi_tc -s 1 -c 1 \
    -o /tmp/$n python tools/prof_one.py multi 32,64,56,56,64 3 --reps 2 --tc > /dev/null 2>&1
ncu -i /tmp/$n.ncu-rep --page raw --csv > gpurun_out/$n.raw.csv 2>/dev/null
ncu -i /tmp/$n.ncu-rep --page source --csv --print-source sass > gpurun_out/$n.src.csv 2>/dev/null
gzip -f gpurun_out/$n.src.csv
ls -la gpurun_out
