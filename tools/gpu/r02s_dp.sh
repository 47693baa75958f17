export PYTHONUNBUFFERED=1
timeout 900 python tools/libab.py 960,3840,5760,7680,9600,11520,15360,19200 variants/base2.so variants/dp.so --rounds 2 --reps 5 > gpurun_out/ab_dp.txt 2>&1
CHOL_LIB_OVERRIDE=variants/dp.so timeout 120 python tools/chain_trace.py 1 5 --list > gpurun_out/chain_N1_dp.txt 2>&1
CHOL_LIB_OVERRIDE=variants/dp.so timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_production.py tests/test_gpu_sched.py tests/test_gpu_dist.py -m gpu -x -q > gpurun_out/pytest_dp.txt 2>&1
