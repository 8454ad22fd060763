#!/bin/bash
# On the GPU box: the session's final evidence -- GPU suite (plain and HRS_FORCE_REDO=1), smoke,
# the reference arm, then micro/evidence_box.sh (bench lines c1..c4, c2 launch list, ncu captures).
export PYTHONPATH=$PWD
tag=${TAG:-r02d}
mkdir -p gpurun_out/ev
python -m pytest tests -m gpu -x -q > gpurun_out/ev/${tag}_gputest.txt 2>&1
HRS_FORCE_REDO=1 python -m pytest tests -m gpu -x -q > gpurun_out/ev/${tag}_gputest_force_redo.txt 2>&1
python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/ev/${tag}_smoke.txt 2>&1
python bench.py --impl reference > gpurun_out/ev/${tag}_bench_reference.json 2> gpurun_out/ev/bench_reference.err
TAG=$tag bash micro/evidence_box.sh
