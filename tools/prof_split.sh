# usage: bash tools/prof_split.sh "K variant size" ... ; full ncu capture of the cluster-split kernel
cd /root/repo
mkdir -p gpurun_out
for spec in "$@"; do set -- $spec
n=prof_split_k$1_v$2_s$3
timeout 300 ncu --set full --clock-control none --import-source on -k regex:k_conv2d_split -s 3 -c 1 \
    -o /tmp/$n python tools/prof_one.py single $3 $1 --reps 4 --variant $2 > /dev/null 2>&1
ncu -i /tmp/$n.ncu-rep --page raw --csv > gpurun_out/$n.raw.csv 2>/dev/null
ncu -i /tmp/$n.ncu-rep --page source --csv --print-source sass > gpurun_out/$n.src.csv 2>/dev/null
gzip -f gpurun_out/$n.src.csv
done
