timeout 900 python -m pytest tests/test_gpu_production.py -m gpu -q -k host_cpu 2>&1 | tail -3
nproc
python tools/hetero_run.py 9600,19200,46080 0,40,24,16,12,8,6
