#!/bin/bash
# iteration: fast GPU parity, per-level traces (C2, C4), short C4 bench
mkdir -p gpurun_out
T=${TAG:-r2b}
timeout 600 python -m pytest tests/test_gpu_parity.py -m "gpu and not slow" -x -q > gpurun_out/${T}_pytest.txt 2>&1
echo "pytest rc=$?" >> gpurun_out/${T}_pytest.txt
timeout 300 python -m pytest tests/test_dist.py -m "gpu" -x -q > gpurun_out/${T}_pytest_dist.txt 2>&1
echo "pytest rc=$?" >> gpurun_out/${T}_pytest_dist.txt
timeout 300 python tools/trace_bfs.py c2 2 > gpurun_out/${T}_trace_c2.txt 2>&1
timeout 600 python bench.py --config c4 --steps 8 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/${T}_bench_c4.json 2> gpurun_out/${T}_bench_c4.err
timeout 600 python tools/trace_bfs.py c4 1 > gpurun_out/${T}_trace_c4.txt 2>&1
