for L in base wa wb; do
  python micro/c1_exp.py $L 22 64 64
  for spec in "and2 64" "and3 64" "and4 64"; do
    timeout 300 python micro/scatter_exp.py run $L $spec
  done
done
