#!/bin/bash
# round-2 first GPU pass: box facts, GPU parity (incl. full-size C2/C3/C4), bench on C4, per-level trace of C4
mkdir -p gpurun_out
(nproc; free -g; lscpu | head -25; nvidia-smi -q | grep -i -A3 "Clocks$" | head -20) > gpurun_out/r2a_box.txt 2>&1
timeout 1500 python -m pytest tests -m gpu -x -q --durations=15 > gpurun_out/r2a_pytest.txt 2>&1
echo "pytest rc=$?" >> gpurun_out/r2a_pytest.txt
timeout 1200 python bench.py --steps 10 --warmup 3 > gpurun_out/r2a_bench.json 2> gpurun_out/r2a_bench.err
echo "bench rc=$?" >> gpurun_out/r2a_bench.err
timeout 900 python tools/trace_bfs.py c4 1 > gpurun_out/r2a_trace_c4.txt 2>&1
