#!/bin/bash
# On the GPU box: ncu --set full of ONE launch of kernel regex $1 (after skipping $2) in
# micro/prof_c2.py, optionally with HRS_LIB=micro/libhrs_$3.so; keeps the per-SASS source
# CSV (executed instructions, stall samples, shared wavefronts) and the raw page under
# gpurun_out/ncu/$4_* for offline reading.
set -u
export PYTHONPATH=$PWD
[ -n "${3:-}" ] && export HRS_LIB=$PWD/micro/libhrs_$3.so
out=gpurun_out/ncu; mkdir -p $out; tag=$4
ncu --set full --import-source on --clock-control none -k "regex:$1" -s $2 -c 1 -f -o $out/$tag \
    python micro/prof_c2.py ${LOG2N:-28} ${DIST:-uniform} > $out/$tag.log 2>&1
python profiles/ncu_summary.py $out/$tag.ncu-rep > $out/${tag}_summary.txt
ncu -i $out/$tag.ncu-rep --page source --csv --print-source sass > $out/${tag}_sass.csv 2> /dev/null
python profiles/ncu_stalls.py $out/${tag}_sass.csv 40 > $out/${tag}_stalls.txt 2>&1
ncu -i $out/$tag.ncu-rep --page raw --csv > $out/${tag}_raw.csv 2> /dev/null
gzip -f $out/${tag}_sass.csv $out/${tag}_raw.csv
rm -f $out/$tag.ncu-rep
