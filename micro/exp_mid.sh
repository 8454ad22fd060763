for L in base mid; do
  python micro/c1_exp.py $L 20 32 0
  python micro/c1_exp.py $L 20 64 64
  python micro/c1_exp.py $L 22 64 64
  for spec in "uniform 32" "and3 32" "uniform 64" "and2 64" "and3 64" "and4 64"; do
    timeout 300 python micro/scatter_exp.py run $L $spec
  done
done
