#!/bin/bash
# ncu full captures of the tensor-core variant (default and a tuning variant) on configs[2]
cd "$(dirname "$0")/.."
mkdir -p gpurun_out
for mv in 0 ${MV:-50}; do
n=prof_tcv${mv}_config2
timeout 300 ncu --set full --clock-control none --import-source on -k regex:k_conv2d_multi_tc -s 1 -c 1 \
    -o /tmp/$n python tools/prof_one.py multi 32,64,56,56,64 3 --reps 2 --tc --mvariant $mv > /dev/null 2>&1
ncu -i /tmp/$n.ncu-rep --page raw --csv > gpurun_out/$n.raw.csv 2>/dev/null
ncu -i /tmp/$n.ncu-rep --page source --csv --print-source sass > gpurun_out/$n.src.csv 2>/dev/null
gzip -f gpurun_out/$n.src.csv
done
