# usage: bash tools/prof_multi.sh "N,C,H,W,F K mvariant" ... ; ncu full capture of the multi kernel
cd /root/repo
mkdir -p gpurun_out
for spec in "$@"; do set -- $spec
n=prof_multi_$(echo $1 | tr ',' 'x')_k$2_mv$3
ncu --set full --clock-control none --import-source on -k regex:k_conv2d_multi -s 1 -c 1 \
    -o /tmp/$n python tools/prof_one.py multi $1 $2 --reps 2 --mvariant $3 > /dev/null 2>&1
ncu -i /tmp/$n.ncu-rep --page raw --csv > gpurun_out/$n.raw.csv 2>/dev/null
ncu -i /tmp/$n.ncu-rep --page source --csv --print-source sass > gpurun_out/$n.src.csv 2>/dev/null
gzip -f gpurun_out/$n.src.csv
done
ls gpurun_out | grep prof_multi
