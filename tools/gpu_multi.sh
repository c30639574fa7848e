#!/bin/bash
# Multi-channel batch on the GPU box (TAG): GPU tests (optionally -k TESTK), smoke, the variant table,
# the multi-channel bench lines (CUDA cores and tensor cores) and ncu captures of the default kernel.
cd "$(dirname "$0")/.."
mkdir -p gpurun_out
TAG=${TAG:-m}
if [ "${SKIP_TESTS:-0}" != "1" ]; then
  timeout 1500 python -m pytest tests -m gpu -q -p no:cacheprovider ${TESTK:+-k "$TESTK"} > gpurun_out/gpu_tests_$TAG.log 2>&1
  echo "gpu tests rc=$?"; tail -3 gpurun_out/gpu_tests_$TAG.log
  timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke_$TAG.log 2>&1
  echo "smoke rc=$?"; tail -1 gpurun_out/smoke_$TAG.log
fi
timeout 600 python tools/multi_variants.py --table1 --variants ${VARIANTS:-0,8,100,101,tc} > gpurun_out/multi_variants_$TAG.txt 2>&1
echo "variants rc=$?"
for wl in config2 config3 table1; do
  timeout 600 python bench.py --workload $wl --steps 10 > gpurun_out/bench_${TAG}_$wl.json 2> gpurun_out/bench_${TAG}_$wl.err
  echo "bench $wl rc=$?"
done
prof() {  # name, kernel regex, prof_one.py args
  local n=$1 k=$2; shift 2
  timeout 600 ncu --set full --clock-control none --import-source on -k regex:$k -s 2 -c 1 -o /tmp/$n \
      python tools/prof_one.py "$@" --reps 3 > /dev/null 2>&1
  ncu -i /tmp/$n.ncu-rep --page raw --csv > gpurun_out/$n.raw.csv 2>/dev/null
  ncu -i /tmp/$n.ncu-rep --page source --csv --print-source sass > gpurun_out/$n.src.csv 2>/dev/null
  gzip -f gpurun_out/$n.src.csv
}
prof ${TAG}_ncu_multi_config3 k_conv2d_mob multi 128,3,224,224,64 7
prof ${TAG}_ncu_multi_config2 k_conv2d_mob multi 32,64,56,56,64 3
prof ${TAG}_ncu_conv11c1 k_conv2d_mob multi 128,1,224,224,64 3
ls gpurun_out | grep $TAG | head -30
