export PYTHONUNBUFFERED=1
timeout 1200 python tools/libab.py 3840,9600,19200 variants/base.so variants/s2.so variants/s1.so variants/s0.so --rounds 2 --reps 5 > gpurun_out/ab4.txt 2>&1
