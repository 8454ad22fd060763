#!/bin/bash
# On the GPU box: time libhrs variants (micro/libhrs_NAME.so) on 2^28 pairs.
#   bash micro/exp_run.sh "name1 name2 ..." "uniform and3" [kbits]
export PYTHONPATH=$PWD
for d in $2; do for v in $1; do timeout 300 python micro/scatter_exp.py run $v $d ${3:-32}; done; done
