export PYTHONUNBUFFERED=1
CHOL_LIB_OVERRIDE=variants/pf2.so timeout 300 python tools/solve_bench.py 19200 960 && CHOL_LIB_OVERRIDE=variants/pf2.so ncu --set full --clock-control none --import-source on -k regex:k_sweep_mma -s 2 -c 1 -o gpurun_out/sweep_mma python tools/solve_bench.py 19200 960 > gpurun_out/ncu_sweep.log 2>&1
