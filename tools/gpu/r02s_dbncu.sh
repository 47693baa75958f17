export PYTHONUNBUFFERED=1
CHOL_SOLVE_RC=48 timeout 300 python tools/solve_bench.py 19200 960 && CHOL_SOLVE_RC=48 ncu --set full --clock-control none --import-source on -k regex:k_sweep_db -s 2 -c 1 -o gpurun_out/sweep_db python tools/solve_bench.py 19200 960 > gpurun_out/ncu_db.log 2>&1
