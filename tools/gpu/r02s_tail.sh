export PYTHONUNBUFFERED=1
timeout 900 python tools/tail_sweep.py 4,5,6,7,8,9,10,11,12,14,16,20 2,3,4,5,6 > gpurun_out/tail_sweep_r02s.txt 2>&1
