for bt in 0 ""; do
  echo "CHOL_BLOCK_TAIL=$bt"
  for R in 2 4; do for n in 7680 9600 19200; do
    if [ -n "$bt" ]; then export CHOL_BLOCK_TAIL=$bt; else unset CHOL_BLOCK_TAIL; fi
    python bench.py --logical-ranks $R --n $n --steps 4 --warmup 2 2>&1 | tail -1 | python -c "import sys,json; d=json.loads(sys.stdin.read()); print(d['logical_ranks'], d['grid'], d['config']['n'], round(d['ms_per_step'],3), round(d['value'],2))"
  done; done
done
