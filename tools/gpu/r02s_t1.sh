export PYTHONUNBUFFERED=1
timeout 900 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_s2.txt 2>&1
timeout 600 python tools/libab.py 46080 variants/base.so variants/s2.so --rounds 2 --reps 3 > gpurun_out/ab5.txt 2>&1
