#!/bin/bash
# Quick state check on the GPU box: GPU tests, default bench line, multi variants incl. the TC variant.
cd "$(dirname "$0")/.."
mkdir -p gpurun_out
TAG=${TAG:-chk}
timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/gpu_tests_$TAG.log 2>&1
echo "gpu tests rc=$?"; tail -3 gpurun_out/gpu_tests_$TAG.log
timeout 600 python bench.py > gpurun_out/bench_$TAG.json 2> gpurun_out/bench_$TAG.err
echo "bench rc=$?"
timeout 300 python tools/multi_variants.py --variants 0,tc > gpurun_out/multi_$TAG.txt 2>&1
echo "multi rc=$?"; cat gpurun_out/multi_$TAG.txt
