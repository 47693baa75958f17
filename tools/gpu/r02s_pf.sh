export PYTHONUNBUFFERED=1
nvcc -gencode arch=compute_100a,code=sm_100a -O3 -std=c++17 -I paper_conf_ipps_agullobehkmt15_b200/csrc -o /tmp/potf2_phases tools/microbench/potf2_phases.cu -lcuda && timeout 60 /tmp/potf2_phases > gpurun_out/potf2_phases_pf.txt 2>&1
timeout 900 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_pf.txt 2>&1
timeout 900 python tools/libab.py 960,3840,7680,9600,11520,19200 variants/s2.so variants/pf.so --rounds 2 --reps 5 > gpurun_out/ab6.txt 2>&1
