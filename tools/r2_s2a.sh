#!/bin/bash
# r2 session-2 first GPU pass: smoke, GPU parity (not slow), default bench (C4), reference arm, C4 launch list
mkdir -p gpurun_out
T=${TAG:-r2s2a}
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv > gpurun_out/${T}_smi.txt 2>&1
nproc >> gpurun_out/${T}_smi.txt
timeout 300 python -c "import __graft_entry__ as e; e.smoke()" > gpurun_out/${T}_smoke.txt 2>&1
echo "smoke rc=$?" >> gpurun_out/${T}_smoke.txt
timeout 1200 python -m pytest tests -m "gpu and not slow" -x -q --timeout 300 > gpurun_out/${T}_pytest.txt 2>&1
echo "pytest rc=$?" >> gpurun_out/${T}_pytest.txt
timeout 1500 python bench.py > gpurun_out/${T}_bench.json 2> gpurun_out/${T}_bench.err
echo "bench rc=$?" >> gpurun_out/${T}_bench.err
timeout 900 python bench.py --impl reference --steps 2 --warmup 1 > gpurun_out/${T}_ref.json 2> gpurun_out/${T}_ref.err
echo "ref rc=$?" >> gpurun_out/${T}_ref.err
timeout 900 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv \
  --log-file gpurun_out/${T}_launches_c4.csv python tools/prof_bfs.py --config c4 --reps 1 > gpurun_out/${T}_launches_c4.log 2>&1
python tools/launches.py gpurun_out/${T}_launches_c4.csv --json gpurun_out/${T}_launches_c4.json > gpurun_out/${T}_launches_c4.txt 2>&1
