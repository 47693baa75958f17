export PYTHONUNBUFFERED=1
timeout 1500 python tools/libab.py 15360,19200,23040,30720 paper_conf_ipps_agullobehkmt15_b200/libchol_b200.so paper_conf_ipps_agullobehkmt15_b200/libchol_b200.so:CHOL_POTRF_BLOCKDAG=1 --rounds 2 --reps 3 > gpurun_out/ab_bd.txt 2>&1
