# Fig 1 / Fig 15 selectivity sweeps (BASELINE config 2) on one B200.
mkdir -p gpurun_out
timeout 1500 python scripts/sweep.py fig1 > gpurun_out/sweep_fig1.jsonl 2> gpurun_out/sweep.err
timeout 1500 python scripts/sweep.py fig15 > gpurun_out/sweep_fig15.jsonl 2>> gpurun_out/sweep.err
