#!/bin/bash
# c1 / c2 with and without the forked local-sort launches (HRS_FORK)
export PYTHONPATH=$PWD
for f in 1 0 1 0; do
  echo "HRS_FORK=$f c1: $(HRS_LIB=$PWD/micro/libhrs_fk.so HRS_FORK=$f python -c "
import torch, gen, paper_1611_01137_b200 as hrs
n=1<<20; k=gen.keys(n,32,'uniform',device='cuda'); ko=torch.empty_like(k)
t=torch.empty(hrs.temp_bytes(n,4,0),dtype=torch.uint8,device='cuda')
for _ in range(5): hrs.sort(k,keys_out=ko,temp=t)
torch.cuda.synchronize(); a,b=torch.cuda.Event(enable_timing=True),torch.cuda.Event(enable_timing=True)
a.record()
for _ in range(200): hrs.sort(k,keys_out=ko,temp=t)
b.record(); torch.cuda.synchronize(); print(round(a.elapsed_time(b)/200,4),'ms')
" 2>&1 | tail -1)"
done
HRS_FORK=1 bash micro/exp_run.sh "fk" "uniform and3"
HRS_FORK=0 bash micro/exp_run.sh "fk" "uniform and3"
