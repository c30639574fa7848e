cd /root/repo; mkdir -p gpurun_out
timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/gpu_tests_s3.log 2>&1; echo "tests rc=$?"; tail -3 gpurun_out/gpu_tests_s3.log
timeout 600 python tools/band_sweep.py --sizes 1024,2048,4096,8192 > gpurun_out/band_sweep_s3.txt 2>&1; echo "band rc=$?"
timeout 300 python tools/small_sizes.py 0 > gpurun_out/small_s3.txt 2>&1
cat gpurun_out/band_sweep_s3.txt gpurun_out/small_s3.txt
