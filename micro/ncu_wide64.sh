#!/bin/bash
# On the GPU box: ncu --set full capture of the wide local sort of 64-bit keys, size class 4
# (k_local<u64, u64, 128, 16, 2, 3, WIDE=1>), second sort of c4 AND-2, summarised under gpurun_out/ncu/.
set -u
export PYTHONPATH=$PWD
out=gpurun_out/ncu
mkdir -p $out
name=wide64_c4
ncu --set full --import-source on --clock-control none --kernel-name-base demangled \
    -k "regex:k_local<unsigned long long, unsigned long long, .int.128, .int.16, .int.2, .int.3, .int.1>" -s 1 -c 1 -f -o $out/$name \
    python micro/prof_sort.py 28 64 ${DIST:-and2} > $out/$name.log 2>&1
python profiles/ncu_summary.py $out/$name.ncu-rep > $out/${name}_summary.txt
ncu -i $out/$name.ncu-rep --page source --csv --print-source cuda,sass > $out/${name}_src.csv 2> /dev/null
python profiles/ncu_lines.py $out/${name}_src.csv 30 > $out/${name}_lines.txt 2>&1
python profiles/ncu_smem.py $out/${name}_src.csv 30 > $out/${name}_smem.txt 2>&1
rm -f $out/$name.ncu-rep $out/${name}_src.csv
