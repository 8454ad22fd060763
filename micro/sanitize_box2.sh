#!/bin/bash
# On the GPU box: compute-sanitizer memcheck / racecheck / synccheck over micro/sanitize_run.py at
# 2^16 and 2^20 (+7) records (2^20: 256 buckets of ~4096 records -> the counting local sort).
export PYTHONPATH=$PWD
export HRS_GRAPHS=0
out=gpurun_out/sanitizer; mkdir -p $out
CS=/usr/local/cuda/bin/compute-sanitizer
for tool in memcheck racecheck synccheck; do
  extra=""; [ $tool = memcheck ] && extra="--leak-check no"; [ $tool = racecheck ] && extra="--racecheck-report all"
  timeout 1500 $CS --tool $tool $extra --print-limit 50 python micro/sanitize_run.py 16 20 > $out/$tool.log 2>&1
  echo "$tool rc=$?" >> $out/$tool.log
done
tail -n 4 $out/*.log
