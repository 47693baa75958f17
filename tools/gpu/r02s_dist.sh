export PYTHONUNBUFFERED=1
B="python bench.py --no-cpu-baseline --no-e2e --no-bounds --no-solve --extra-n 0 --steps 3 --warmup 2"
for cfg in "1 19200 1x2" "2 19200 2x2" "3 38400 2x4" "1 9600 1x2"; do
  set -- $cfg; R=$((2**$1)); n=$2; g=$3
  timeout 300 $B --n $n --logical-ranks $R --grid $g | tail -1
done > gpurun_out/dist_proxy_r02s.txt 2>&1
