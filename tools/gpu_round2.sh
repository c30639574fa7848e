#!/bin/bash
# One round-2 measurement batch on the GPU box (outputs under gpurun_out/ with TAG):
# GPU tests + smoke, the default bench line (sweep, batch 8), the other workloads' bench lines (both
# multi-channel implementations), the reference (oracle) arm, the ncu launch list of the default bench
# command, and ncu --set full captures of the dominant and the other key kernels.
cd "$(dirname "$0")/.."
mkdir -p gpurun_out
TAG=${TAG:-r02}
if [ "${SKIP_TESTS:-0}" != "1" ]; then
  timeout 1500 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/gpu_tests_$TAG.log 2>&1
  echo "gpu tests rc=$?"; tail -3 gpurun_out/gpu_tests_$TAG.log
  timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke_$TAG.log 2>&1
  echo "smoke rc=$?"
fi
timeout 900 python bench.py > gpurun_out/bench_$TAG.json 2> gpurun_out/bench_$TAG.err
echo "bench rc=$?"
if [ "${SKIP_WORKLOADS:-0}" != "1" ]; then
  timeout 600 python bench.py --batch 1 --no-e2e --no-cpu-baseline > gpurun_out/bench_${TAG}_b1.json 2> gpurun_out/bench_${TAG}_b1.err
  for wl in config0 config2 config3 config4 table1 pad halo; do
    timeout 600 python bench.py --workload $wl --steps 10 > gpurun_out/bench_${TAG}_$wl.json 2> gpurun_out/bench_${TAG}_$wl.err
    echo "bench $wl rc=$?"
  done
  for wl in config2 config3 table1; do
    timeout 600 python bench.py --workload $wl --steps 10 --multi-impl tc > gpurun_out/bench_${TAG}_${wl}_tc.json 2> gpurun_out/bench_${TAG}_${wl}_tc.err
    echo "bench $wl tc rc=$?"
  done
  timeout 900 python bench.py --impl reference --steps 3 --warmup 3 > gpurun_out/bench_${TAG}_reference.json 2> gpurun_out/bench_${TAG}_reference.err
  echo "bench reference rc=$?"
fi
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_$TAG.csv \
    python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu-baseline > /dev/null 2>&1
echo "ncu launches rc=$?"
prof() {  # name, kernel regex, prof_one.py args
  local n=$1 k=$2; shift 2
  timeout 600 ncu --set full --clock-control none --import-source on -k regex:$k -s 2 -c 1 -o /tmp/$n \
      python tools/prof_one.py "$@" --reps 3 > /dev/null 2>&1
  ncu -i /tmp/$n.ncu-rep --page raw --csv > gpurun_out/$n.raw.csv 2>/dev/null
  ncu -i /tmp/$n.ncu-rep --page source --csv --print-source sass > gpurun_out/$n.src.csv 2>/dev/null
  gzip -f gpurun_out/$n.src.csv
}
prof prof_k15_b8_s8192 "k_conv2d_(single|wide|pair)" single 8192 15 --batch 8
prof prof_k3_b8_s8192 "k_conv2d_(single|wide)" single 8192 3 --batch 8
prof prof_k7_b8_s8192 "k_conv2d_(single|wide|pair)" single 8192 7 --batch 8
prof prof_k15_s4096 "k_conv2d_(single|wide)" single 4096 15
prof prof_k5_s2048 "k_conv2d_(single|wide)" single 2048 5
prof prof_direct_k3_s8192 k_conv2d_direct single 8192 3 --direct
prof prof_split_k15_s1024 k_conv2d_split single 1024 15
prof prof_conv11c1 "k_conv2d_(mob|multi2)" multi 128,1,224,224,64 3
prof prof_multi_config3 "k_conv2d_(mob|multi2)" multi 128,3,224,224,64 7
prof prof_tc_config2 k_conv2d_multi_tc multi 32,64,56,56,64 3 --tc
prof prof_tc_config3 k_conv2d_multi_tc multi 128,3,224,224,64 7 --tc
prof prof_config0 "k_conv2d_(single|wide)" single 256 3
ls -la gpurun_out | tail -40
