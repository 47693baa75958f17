export PYTHONUNBUFFERED=1
timeout 1500 python tools/libab.py 19200,46080 variants/cur2.so variants/fr1.so variants/fr2.so --rounds 2 --reps 3 > gpurun_out/ab_fr.txt 2>&1
