cd /root/repo; mkdir -p gpurun_out
n=prof_conv11c1
timeout 300 ncu --set full --clock-control none --import-source on -k regex:k_conv2d_multi -s 1 -c 1 -o /tmp/$n \
  python tools/prof_one.py multi 128,1,224,224,64 3 --reps 2 > /dev/null 2>&1
ncu -i /tmp/$n.ncu-rep --page raw --csv > gpurun_out/$n.raw.csv 2>/dev/null
ncu -i /tmp/$n.ncu-rep --page source --csv --print-source sass > gpurun_out/$n.src.csv 2>/dev/null; gzip -f gpurun_out/$n.src.csv
bash tools/prof2.sh "7 0 8192"
