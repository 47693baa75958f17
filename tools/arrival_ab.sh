for r in 1 2; do for m in 0 1; do
CHOL_ARRIVAL=$m python bench.py --no-cpu-baseline --no-bounds --steps 3 --warmup 3 | python -c "import json,sys; d=json.loads(sys.stdin.readline()); print('arrival $m', round(d['value'],3), 'e2e', round(d['e2e']['value'],3), round(d['e2e']['ms_per_step'],2))"
done; done
CHOL_ARRIVAL=1 timeout 600 python -m pytest tests/test_gpu_parity.py -q -x -k "host_pointers or lower_only" 2>&1 | tail -2
