export PYTHONUNBUFFERED=1
timeout 900 python tools/libab.py 3840,19200 variants/base.so variants/new.so variants/pre0.so variants/pre1.so --rounds 2 --reps 5 > gpurun_out/ab2.txt 2>&1
for v in base new pre0; do CHOL_LIB_OVERRIDE=variants/$v.so timeout 100 python tools/job_trace.py 19200 > gpurun_out/jt_$v.json 2>&1; done
