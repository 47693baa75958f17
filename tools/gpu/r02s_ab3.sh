export PYTHONUNBUFFERED=1
timeout 900 python tools/libab.py 19200 variants/base.so variants/new.so variants/vsmem.so variants/vbloat.so --rounds 2 --reps 5 > gpurun_out/ab3.txt 2>&1
