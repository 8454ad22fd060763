#!/bin/bash
# On the GPU box: the ncu launch list of one bench.py c2 run (cold-cache, serialised --
# compare shares, not absolute times) and full captures of both scatter passes of the
# last sort (DRAM traffic per launch for bench.py's roofline.traffic).
export PYTHONPATH=$PWD
out=gpurun_out/prof; mkdir -p $out
cfg=${CFG:-c2}
ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv \
    --log-file $out/launches_$cfg.csv python bench.py --config $cfg --steps 2 --warmup 3 > $out/launches_$cfg.log 2>&1
python micro/launch_summary.py $out/launches_$cfg.csv > $out/launches_${cfg}_summary.txt
# the scatter launches of the second sort (passes 1 and 2 carry the records)
nsc=${NSC:-4}
ncu --set full --clock-control none -k regex:k_scatter -s $nsc -c 2 -f -o $out/sc_$cfg \
    python micro/prof_c2.py 28 uniform > $out/sc_$cfg.log 2>&1
python profiles/ncu_summary.py $out/sc_$cfg.ncu-rep > $out/sc_${cfg}_summary.txt
rm -f $out/sc_$cfg.ncu-rep
