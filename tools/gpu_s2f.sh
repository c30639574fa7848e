#!/bin/bash
cd "$(dirname "$0")/.."
mkdir -p gpurun_out
PROF=1 VARIANTS=0,tc,tc22,tc24 bash tools/tc_check.sh
timeout 600 python tools/band_sweep.py > gpurun_out/band_sweep.txt 2>&1; cat gpurun_out/band_sweep.txt
timeout 300 python tools/band_sweep.py --sizes 2048,4096 --ks 7,9,11,13,15 --variant 9 > gpurun_out/band_sweep_v9.txt 2>&1; cat gpurun_out/band_sweep_v9.txt
timeout 300 python tools/gpu_side_calls.py > gpurun_out/gpu_side_calls.txt 2>&1; cat gpurun_out/gpu_side_calls.txt
