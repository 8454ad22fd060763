#!/bin/bash
# On the GPU box: compute-sanitizer memcheck / racecheck / synccheck over micro/sanitize_run.py.
export PYTHONPATH=$PWD
export HRS_GRAPHS=0
out=gpurun_out/sanitizer; mkdir -p $out
CS=/usr/local/cuda/bin/compute-sanitizer
$CS --tool memcheck --leak-check no --print-limit 50 python micro/sanitize_run.py 16 20 > $out/memcheck.log 2>&1; echo "memcheck rc=$?" >> $out/memcheck.log
$CS --tool racecheck --racecheck-report all --print-limit 50 python micro/sanitize_run.py 16 > $out/racecheck.log 2>&1; echo "racecheck rc=$?" >> $out/racecheck.log
$CS --tool synccheck --print-limit 50 python micro/sanitize_run.py 16 > $out/synccheck.log 2>&1; echo "synccheck rc=$?" >> $out/synccheck.log
tail -n 4 $out/*.log
