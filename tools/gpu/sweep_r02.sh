set -x
python tools/sweep.py 4,6,8,10,12,16,20,24,32,48 > gpurun_out/sweep_r02.jsonl 2> gpurun_out/sweep_r02.err
python tools/ablation.py 28800 > gpurun_out/ablation_r02.jsonl 2>> gpurun_out/sweep_r02.err
python tools/big_run.py 92160 > gpurun_out/big_n92160_r02.json 2>> gpurun_out/sweep_r02.err
tail -3 gpurun_out/sweep_r02.err
