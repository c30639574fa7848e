#!/bin/bash
# ncu --set full captures (raw + SASS source pages) of the default single-channel kernels of given
# sweep points: SPECS="size:K[:batch] ..." (TAG prefix)
cd "$(dirname "$0")/.."
mkdir -p gpurun_out
TAG=${TAG:-sp}
for spec in $SPECS; do
  IFS=: read S K B <<< "$spec"
  n=${TAG}_s${S}_k${K}_b${B:-8}
  timeout 600 ncu --set full --clock-control none --import-source on -k regex:"k_conv2d_(single|wide|pair|split)" -s 2 -c 1 -o /tmp/$n \
      python tools/prof_one.py single $S $K --batch ${B:-8} --reps 3 ${VARIANT:+--variant $VARIANT} > /dev/null 2>&1
  ncu -i /tmp/$n.ncu-rep --page raw --csv > gpurun_out/$n.raw.csv 2>/dev/null
  ncu -i /tmp/$n.ncu-rep --page source --csv --print-source sass > gpurun_out/$n.src.csv 2>/dev/null
  gzip -f gpurun_out/$n.src.csv
done
