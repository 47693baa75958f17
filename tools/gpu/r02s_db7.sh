export PYTHONUNBUFFERED=1
for lib in dbA dbu8 dbu24; do echo $lib; CHOL_LIB_OVERRIDE=variants/$lib.so timeout 300 python tools/solve_bench.py 19200 96,960; CHOL_LIB_OVERRIDE=variants/$lib.so timeout 300 python tools/solve_bench.py 46080 960; done > gpurun_out/solve_db7.txt 2>&1
