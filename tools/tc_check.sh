#!/bin/bash
# tensor-core variant: parity tests, timings vs the CUDA-core kernel, one ncu capture on configs[2]
cd "$(dirname "$0")/.."
mkdir -p gpurun_out
timeout 300 python -m pytest tests/test_gpu_multi.py -q -p no:cacheprovider -k tensor_core -x 2>&1 | tail -15 > gpurun_out/tc_tests.txt
cat gpurun_out/tc_tests.txt
timeout 300 python tools/multi_variants.py --variants ${VARIANTS:-0,tc} > gpurun_out/tc_multi.txt 2>&1; cat gpurun_out/tc_multi.txt
if [ "${PROF:-0}" = "1" ]; then
n=prof_tc4_config2
timeout 300 ncu --set full --clock-control none --import-source on -k regex:k_conv2d_multi_tc -s 1 -c 1 \
    -o /tmp/$n python tools/prof_one.py multi 32,64,56,56,64 3 --reps 2 --tc > /dev/null 2>&1
ncu -i /tmp/$n.ncu-rep --page raw --csv > gpurun_out/$n.raw.csv 2>/dev/null
ncu -i /tmp/$n.ncu-rep --page source --csv --print-source sass > gpurun_out/$n.src.csv 2>/dev/null
gzip -f gpurun_out/$n.src.csv
fi
