export PYTHONUNBUFFERED=1 CHAIN_TB=90
timeout 120 python tools/chain_trace.py 10 3 --list > gpurun_out/chain_N10.txt 2>&1; echo rc=$? >> gpurun_out/chain_N10.txt
for N in 8 12 16 20; do timeout 100 python tools/chain_trace.py $N 3; done > gpurun_out/chain_Ns.txt 2>&1
timeout 300 python tools/sweep.py 8,10,12 > gpurun_out/sweep_small.jsonl 2>&1
nvcc -gencode arch=compute_100a,code=sm_100a -O3 -std=c++17 -I paper_conf_ipps_agullobehkmt15_b200/csrc -o /tmp/potf2_phases tools/microbench/potf2_phases.cu -lcuda && timeout 60 /tmp/potf2_phases > gpurun_out/potf2_phases.txt 2>&1
