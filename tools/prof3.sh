# usage: bash tools/prof3.sh "K variant size kernel_regex [tag]" ... ; ncu --set full of one conv2d_single launch
# per spec (raw + SASS-source CSVs into gpurun_out/). Run under gpurun, one GPU.
cd "$(dirname "$0")/.."
mkdir -p gpurun_out
for spec in "$@"; do set -- $spec
n=prof_${5:-k$1_v$2_s$3}
timeout 600 ncu --set full --clock-control none --import-source on -k regex:$4 -s 3 -c 1 \
    -o /tmp/$n python tools/prof_one.py single $3 $1 --reps 4 --variant $2 > /dev/null 2>&1
ncu -i /tmp/$n.ncu-rep --page raw --csv > gpurun_out/$n.raw.csv 2>/dev/null
ncu -i /tmp/$n.ncu-rep --page source --csv --print-source sass > gpurun_out/$n.src.csv 2>/dev/null
gzip -f gpurun_out/$n.src.csv
done
