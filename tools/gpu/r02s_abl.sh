export PYTHONUNBUFFERED=1
timeout 900 python tools/ablation.py 28800 > gpurun_out/ablation_r02s.jsonl 2> gpurun_out/ablation_r02s.err
timeout 600 python tools/big_run.py 92160 > gpurun_out/big_n92160_r02s.json 2>> gpurun_out/ablation_r02s.err
