#!/bin/bash
# On the GPU box: the round's evidence -- bench lines (c1..c4), the ncu launch list of c2 and
# full captures of the hot kernels (scatter, counting local sort, histogram), summarised.
export PYTHONPATH=$PWD
tag=${TAG:-r02}
out=gpurun_out/ev; mkdir -p $out
python bench.py > $out/${tag}_bench_c2.json 2> $out/bench_c2.err
for c in c1 c4; do python bench.py --config $c --no-cpu > $out/${tag}_bench_$c.json 2> $out/bench_$c.err; done
for d in and2 and3 and4 const; do python bench.py --config c3 --dist $d --no-cpu --no-e2e > $out/${tag}_bench_c3_$d.json 2>&1; done
for d in and2 and4 const; do python bench.py --config c4 --dist $d --no-cpu --no-e2e > $out/${tag}_bench_c4_$d.json 2>&1; done
ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv \
    --log-file $out/launches_c2.csv python bench.py --steps 2 --warmup 3 --no-cpu --no-e2e > $out/launches_c2.log 2>&1
python micro/launch_summary.py $out/launches_c2.csv > $out/${tag}_launches_c2_summary.txt
# full captures of the second sort's hot kernels
for spec in "k_scatter 4 2 sc" "k_local_cnt 2 2 loc" "k_hist 4 2 hist"; do
    set -- $spec
    bash micro/ncu_one.sh $1 $2 $3 "" ${tag}_$4
    mv gpurun_out/ncu/${tag}_$4_* $out/ 2>/dev/null
done
ls -la $out
