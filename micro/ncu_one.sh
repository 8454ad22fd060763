#!/bin/bash
# On the GPU box: ncu --set full of kernel regex $1 (skip $2 launches, capture $3) in micro/prof_c2.py
# (optionally with HRS_LIB=micro/libhrs_$4.so), summaries under gpurun_out/ncu/$5_*
set -u
export PYTHONPATH=$PWD
[ -n "${4:-}" ] && export HRS_LIB=$PWD/micro/libhrs_$4.so
out=gpurun_out/ncu; mkdir -p $out; tag=$5
ncu --set full --import-source on --clock-control none -k "regex:$1" -s $2 -c $3 -f -o $out/$tag \
    python micro/prof_c2.py ${LOG2N:-28} ${DIST:-uniform} > $out/$tag.log 2>&1
python profiles/ncu_summary.py $out/$tag.ncu-rep > $out/${tag}_summary.txt
ncu -i $out/$tag.ncu-rep --page source --csv --print-source cuda,sass > $out/${tag}_src.csv 2> /dev/null
python profiles/ncu_smem.py $out/${tag}_src.csv 40 > $out/${tag}_smem.txt
python profiles/ncu_lines.py $out/${tag}_src.csv 40 > $out/${tag}_lines.txt 2>&1
ncu -i $out/$tag.ncu-rep --page raw --csv | python -c "
import csv,sys
r=list(csv.reader(sys.stdin)); h=r[0]
for row in r[2:]:
  for i,n in enumerate(h):
    if any(k in n for k in ('lsu_wavefronts','dram__bytes','smsp__inst_executed.sum','gpu__time_duration','l1tex__t_sectors_pipe_lsu_mem_global_op_st.sum','l1tex__data_bank','smsp__warp_issue_stalled')):
        print(n, row[i], r[1][i])
  print('----')
" > $out/${tag}_raw.txt
rm -f $out/$tag.ncu-rep $out/${tag}_src.csv
