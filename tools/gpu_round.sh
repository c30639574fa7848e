#!/bin/bash
# One measurement batch on the GPU box: GPU tests, bench line, ncu launch list of the bench command,
# ncu full captures (raw + source CSV) of the dominant kernel and of the HBM-bound kernel, and of the
# Fig. 1a direct baseline for the memory-transaction comparison. Outputs under gpurun_out/.
cd "$(dirname "$0")/.."
mkdir -p gpurun_out
TAG=${TAG:-r01}
if [ "${SKIP_TESTS:-0}" != "1" ]; then
  timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/gpu_tests_$TAG.log 2>&1
  echo "gpu tests rc=$?"; tail -3 gpurun_out/gpu_tests_$TAG.log
fi
python bench.py > gpurun_out/bench_$TAG.json 2> gpurun_out/bench_$TAG.err
echo "bench rc=$?"
ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_$TAG.csv \
    python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu-baseline > /dev/null 2>&1
echo "ncu launches rc=$?"
for spec in "15 0 8192" "3 0 8192"; do bash tools/prof2.sh "$spec" > /dev/null 2>&1; done
ncu --set full --clock-control none -k regex:k_conv2d_direct -s 3 -c 1 -o /tmp/prof_direct \
    python tools/prof_one.py single 8192 3 --reps 4 --direct > /dev/null 2>&1
ncu -i /tmp/prof_direct.ncu-rep --page raw --csv > gpurun_out/prof_direct_k3_s8192.raw.csv 2>/dev/null
ls -la gpurun_out
