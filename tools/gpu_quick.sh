#!/bin/bash
# Quick check on the GPU box: GPU tests (optionally a -k filter), smoke, the default bench line and
# the single-image sweep (--batch 1, round-1 comparable). Outputs under gpurun_out/ with TAG.
cd "$(dirname "$0")/.."
mkdir -p gpurun_out
TAG=${TAG:-q}
if [ "${SKIP_TESTS:-0}" != "1" ]; then
  timeout ${TEST_TIMEOUT:-1200} python -m pytest tests -m gpu -q -p no:cacheprovider -x ${TESTK:+-k "$TESTK"} > gpurun_out/gpu_tests_$TAG.log 2>&1
  echo "gpu tests rc=$?"; tail -5 gpurun_out/gpu_tests_$TAG.log
  timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke_$TAG.log 2>&1
  echo "smoke rc=$?"; tail -2 gpurun_out/smoke_$TAG.log
fi
timeout 900 python bench.py > gpurun_out/bench_$TAG.json 2> gpurun_out/bench_$TAG.err
echo "bench rc=$?"; tail -3 gpurun_out/bench_$TAG.err
timeout 600 python bench.py --batch 1 --no-e2e --no-cpu-baseline > gpurun_out/bench_${TAG}_b1.json 2> gpurun_out/bench_${TAG}_b1.err
echo "bench b1 rc=$?"; tail -3 gpurun_out/bench_${TAG}_b1.err
for wl in ${WORKLOADS:-}; do
  timeout 600 python bench.py --workload $wl --steps 10 > gpurun_out/bench_${TAG}_$wl.json 2> gpurun_out/bench_${TAG}_$wl.err
  echo "bench $wl rc=$?"; tail -2 gpurun_out/bench_${TAG}_$wl.err
done
