# usage: bash tools/prof2.sh "K variant [size]" ... ; full ncu capture of conv2d_single per spec.
# Exports raw + SASS-source CSVs on the box (small); the .ncu-rep stays in /tmp unless KEEP_REP=1.
cd /root/repo
mkdir -p gpurun_out
for spec in "$@"; do set -- $spec
S=${3:-8192}
n=prof_k$1_v$2_s$S
ncu --set full --clock-control none --import-source on -k regex:k_conv2d_single -s 3 -c 1 \
    -o /tmp/$n python tools/prof_one.py single $S $1 --reps 4 --variant $2 > /dev/null 2>&1
ncu -i /tmp/$n.ncu-rep --page raw --csv > gpurun_out/$n.raw.csv 2>/dev/null
ncu -i /tmp/$n.ncu-rep --page source --csv --print-source sass > gpurun_out/$n.src.csv 2>/dev/null
gzip -f gpurun_out/$n.src.csv
if [ "${KEEP_REP:-0}" = "1" ]; then cp /tmp/$n.ncu-rep gpurun_out/; fi
done
ls -la gpurun_out
