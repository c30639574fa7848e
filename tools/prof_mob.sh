#!/bin/bash
# ncu --set full captures of the filter-blocked multi-channel kernel (tuning variants) on the BASELINE
# multi-channel configs; raw + SASS-source pages under gpurun_out/ with TAG.
cd "$(dirname "$0")/.."
mkdir -p gpurun_out
TAG=${TAG:-mob}
prof() {  # name, kernel regex, prof_one.py args
  local n=$1 k=$2; shift 2
  timeout 600 ncu --set full --clock-control none --import-source on -k regex:$k -s 2 -c 1 -o /tmp/$n \
      python tools/prof_one.py "$@" --reps 3 > /dev/null 2>&1
  ncu -i /tmp/$n.ncu-rep --page raw --csv > gpurun_out/$n.raw.csv 2>/dev/null
  ncu -i /tmp/$n.ncu-rep --page source --csv --print-source sass > gpurun_out/$n.src.csv 2>/dev/null
  gzip -f gpurun_out/$n.src.csv
}
for spec in ${SPECS:-"config3:128,3,224,224,64:7:110" "config2:32,64,56,56,64:3:110"}; do
  IFS=: read nm shape k mv <<< "$spec"
  prof ${TAG}_${nm}_v$mv "k_conv2d_mob" multi $shape $k --mvariant $mv
done
ls gpurun_out | grep $TAG
