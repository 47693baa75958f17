export PYTHONUNBUFFERED=1
for lib in mA mB; do echo $lib; CHOL_LIB_OVERRIDE=variants/$lib.so timeout 300 python tools/solve_bench.py 19200 2,16,32,64; CHOL_LIB_OVERRIDE=variants/$lib.so timeout 300 python tools/solve_bench.py 46080 32; done > gpurun_out/solve_m.txt 2>&1
