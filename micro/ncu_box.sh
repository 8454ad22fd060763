#!/bin/bash
# On the GPU box: ncu --set full captures of the c2 hot kernels (second sort), summarised to text
# under gpurun_out/ncu/ (the .ncu-rep files are deleted: too large to bring back).
#   bash micro/ncu_box.sh [tag] [log2 n] [dist]
set -u
tag=${1:-cur}
export PYTHONPATH=$PWD
out=gpurun_out/ncu
mkdir -p $out
cap() {  # name regex skip   (one sort = 1 init + 4 hist/classify/scatter + 9 local launches for c2)
    ncu --set full --import-source on --clock-control none -k "regex:$2" -s $3 -c 1 -f -o $out/$1 \
        python micro/prof_c2.py ${LOG2N:-28} ${DIST:-uniform} > $out/$1.log 2>&1
    python profiles/ncu_summary.py $out/$1.ncu-rep > $out/${tag}_$1_summary.txt
    ncu -i $out/$1.ncu-rep --page source --csv --print-source cuda,sass > $out/$1_src.csv 2> $out/$1_src.err; head -c 3000 $out/$1_src.csv > $out/$1_src_head.txt
    python profiles/ncu_smem.py $out/$1_src.csv 40 > $out/${tag}_$1_smem.txt
    python profiles/ncu_lines.py $out/$1_src.csv 40 > $out/${tag}_$1_lines.txt 2>&1
    ncu -i $out/$1.ncu-rep --page source --csv --print-source sass > $out/$1_sass.csv 2>/dev/null
    python profiles/ncu_stalls.py $out/$1_sass.csv 40 > $out/${tag}_$1_stalls.txt 2>&1
    rm -f $out/$1_sass.csv
    ncu -i $out/$1.ncu-rep --page raw --csv | python -c "
import csv,sys
r=list(csv.reader(sys.stdin)); h=r[0]
for i,n in enumerate(h):
    if any(k in n for k in ('lsu_wavefronts','data_pipe','dram__bytes','dram__throughput','l1tex__t_sectors_pipe_lsu_mem_global_op_st','l1tex__t_requests_pipe_lsu_mem_global_op_st','smsp__inst_executed_op','sm__cycles_elapsed.avg','gpc__cycles_elapsed.max','smsp__cycles_active')):
        print(n, r[2][i], r[1][i])
" > $out/${tag}_$1_raw.txt
    rm -f $out/$1.ncu-rep $out/$1_src.csv
}
if [ -n "${ONLY:-}" ]; then eval "$ONLY"; exit 0; fi
cap sc k_scatter 4
cap loc5 k_local_cnt 2
cap loc6 k_local_cnt 3
cap hist k_hist 4
ls -la $out
