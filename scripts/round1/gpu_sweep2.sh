# Fig 16 (selective FK join strategies) and Fig 14 (multi-column lookup layouts) sweeps on one B200.
mkdir -p gpurun_out
timeout 1500 python scripts/sweep.py fig16 > gpurun_out/sweep_fig16.jsonl 2> gpurun_out/sweep2.err
timeout 1500 python scripts/sweep.py fig14 > gpurun_out/sweep_fig14.jsonl 2>> gpurun_out/sweep2.err
