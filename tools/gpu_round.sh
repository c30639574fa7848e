#!/bin/bash
# One measurement batch on the GPU box: GPU tests, the default bench line, bench lines of the other
# workloads (both multi-channel implementations), the reference (oracle) arm, the ncu launch list of
# the default bench command, and ncu full captures (raw + SASS-source CSV) of the dominant kernel,
# the HBM-bound kernel, the Fig. 1a direct baseline and the tensor-core variant. Outputs under gpurun_out/.
cd "$(dirname "$0")/.."
mkdir -p gpurun_out
TAG=${TAG:-r01}
if [ "${SKIP_TESTS:-0}" != "1" ]; then
  timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/gpu_tests_$TAG.log 2>&1
  echo "gpu tests rc=$?"; tail -3 gpurun_out/gpu_tests_$TAG.log
fi
timeout 900 python bench.py > gpurun_out/bench_$TAG.json 2> gpurun_out/bench_$TAG.err
echo "bench rc=$?"
if [ "${SKIP_WORKLOADS:-0}" != "1" ]; then
  for wl in config0 config2 config3 config4 table1 pad halo; do
    timeout 600 python bench.py --workload $wl --steps 10 > gpurun_out/bench_${TAG}_$wl.json 2> gpurun_out/bench_${TAG}_$wl.err
    echo "bench $wl rc=$?"
  done
  for wl in config2 config3 table1; do
    timeout 600 python bench.py --workload $wl --steps 10 --multi-impl tc > gpurun_out/bench_${TAG}_${wl}_tc.json 2> gpurun_out/bench_${TAG}_${wl}_tc.err
    echo "bench $wl tc rc=$?"
  done
  timeout 600 python bench.py --impl reference --steps 3 --warmup 3 > gpurun_out/bench_${TAG}_reference.json 2> gpurun_out/bench_${TAG}_reference.err
  echo "bench reference rc=$?"
fi
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_$TAG.csv \
    python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu-baseline > /dev/null 2>&1
echo "ncu launches rc=$?"
for spec in "15 0 8192" "3 0 8192" "7 0 8192"; do timeout 600 bash tools/prof2.sh "$spec" > /dev/null 2>&1; done
# the filter-row split kernel (default for W <= 1024, K >= 11) and the Table I CONV11 C1 multi kernel
timeout 300 ncu --set full --clock-control none --import-source on -k regex:k_conv2d_split -s 3 -c 1 -o /tmp/prof_split \
    python tools/prof_one.py single 1024 15 --reps 4 > /dev/null 2>&1
ncu -i /tmp/prof_split.ncu-rep --page raw --csv > gpurun_out/prof_split_k15_s1024.raw.csv 2>/dev/null
timeout 300 ncu --set full --clock-control none --import-source on -k regex:k_conv2d_multi -s 1 -c 1 -o /tmp/prof_conv11c1 \
    python tools/prof_one.py multi 128,1,224,224,64 3 --reps 2 > /dev/null 2>&1
ncu -i /tmp/prof_conv11c1.ncu-rep --page raw --csv > gpurun_out/prof_conv11c1.raw.csv 2>/dev/null
timeout 300 ncu --set full --clock-control none -k regex:k_conv2d_direct -s 3 -c 1 -o /tmp/prof_direct \
    python tools/prof_one.py single 8192 3 --reps 4 --direct > /dev/null 2>&1
ncu -i /tmp/prof_direct.ncu-rep --page raw --csv > gpurun_out/prof_direct_k3_s8192.raw.csv 2>/dev/null
for spec in "config2 32,64,56,56,64 3" "config3 128,3,224,224,64 7"; do set -- $spec
  n=prof_tc_$1
  timeout 300 ncu --set full --clock-control none --import-source on -k regex:k_conv2d_multi_tc -s 1 -c 1 \
      -o /tmp/$n python tools/prof_one.py multi $2 $3 --reps 2 --tc > /dev/null 2>&1
  ncu -i /tmp/$n.ncu-rep --page raw --csv > gpurun_out/$n.raw.csv 2>/dev/null
  ncu -i /tmp/$n.ncu-rep --page source --csv --print-source sass > gpurun_out/$n.src.csv 2>/dev/null
  gzip -f gpurun_out/$n.src.csv
done
ls -la gpurun_out
