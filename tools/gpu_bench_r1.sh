#!/bin/bash
# round-1 measurement batch: bench line, quick per-K timings, ncu launch list, ncu full captures
cd "$(dirname "$0")/.."
mkdir -p gpurun_out
python bench.py > gpurun_out/bench.json 2> gpurun_out/bench.err
echo "bench rc=$?"
cat gpurun_out/bench.json
for K in 3 5 7 15; do python tools/prof_one.py single 8192 $K --time; done > gpurun_out/quick.txt 2>&1
python tools/prof_one.py single 8192 3 --time --direct >> gpurun_out/quick.txt 2>&1
python tools/prof_one.py multi 32,64,56,56,64 3 --time >> gpurun_out/quick.txt 2>&1
python tools/prof_one.py multi 128,3,224,224,64 7 --time >> gpurun_out/quick.txt 2>&1
cat gpurun_out/quick.txt
ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches.csv \
    python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/bench_ncu.json 2>&1
echo "ncu launches rc=$?"
ncu --set full --clock-control none --import-source on -k regex:k_conv2d_single -s 3 -c 1 \
    -o gpurun_out/prof_k15 python tools/prof_one.py single 8192 15 --reps 4 > /dev/null 2>&1
ncu --set full --clock-control none --import-source on -k regex:k_conv2d_single -s 3 -c 1 \
    -o gpurun_out/prof_k3 python tools/prof_one.py single 8192 3 --reps 4 > /dev/null 2>&1
ncu --set full --clock-control none --import-source on -k regex:k_conv2d_direct -s 3 -c 1 \
    -o gpurun_out/prof_direct_k3 python tools/prof_one.py single 8192 3 --reps 4 --direct > /dev/null 2>&1
ls -la gpurun_out
