export PYTHONUNBUFFERED=1
for i in 1 2; do variants/bin/solve_phases; variants/bin/solve_phases_lk; done > gpurun_out/solve_block_lk.txt 2>&1
timeout 900 python tools/libab.py 960,3840,7680,9600,11520,19200 variants/pf2.so variants/lk.so --rounds 2 --reps 5 > gpurun_out/ab_lk.txt 2>&1
CHOL_LIB_OVERRIDE=variants/lk.so timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_production.py tests/test_gpu_fullsize.py -m gpu -x -q > gpurun_out/pytest_lk.txt 2>&1
