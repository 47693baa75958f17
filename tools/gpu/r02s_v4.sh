export PYTHONUNBUFFERED=1
for i in 1 2; do variants/bin/pt_old; variants/bin/pt_v3; variants/bin/pt_v4; done > gpurun_out/potf2_total_v4.txt 2>&1
variants/bin/pp2_v4 > gpurun_out/pp2_v4.txt 2>&1
timeout 600 python -m pytest tests/test_gpu_parity.py tests/test_gpu_production.py -m gpu -x -q > gpurun_out/pytest_v4.txt 2>&1
timeout 900 python tools/libab.py 960,3840,7680,9600,19200 variants/pf.so variants/v4.so --rounds 2 --reps 5 > gpurun_out/ab8.txt 2>&1
