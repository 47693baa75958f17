B="python bench.py --no-cpu-baseline --no-e2e --no-bounds --steps 3 --warmup 2"
for cfg in "1 24000 1x2" "2 30720 2x2" "3 38400 2x4"; do
  set -- $cfg; R=$((2**$1)); n=$2; g=$3
  $B --n $n | python -c "import json,sys; d=json.loads(sys.stdin.readline()); print('single', $n, round(d['value'],2), round(d['ms_per_step'],2))"
  $B --n $n --logical-ranks $R --grid $g | python -c "import json,sys; d=json.loads(sys.stdin.readline()); print('logical', $R, '$g', $n, round(d['value'],2), round(d['ms_per_step'],2))"
  CHOL_POTRF_BLOCKDAG=0 $B --n $n --logical-ranks $R --grid $g | python -c "import json,sys; d=json.loads(sys.stdin.readline()); print('logical-noblockdag', $R, '$g', $n, round(d['value'],2), round(d['ms_per_step'],2))"
done
