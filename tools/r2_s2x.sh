#!/bin/bash
# full build: GPU parity (not slow), bench (C4) + reference arm, BC timing + launch list on C3, C4 trace
mkdir -p gpurun_out
T=${TAG:-r2s2x}
timeout 300 python -c "import __graft_entry__ as e; e.smoke()" > gpurun_out/${T}_smoke.txt 2>&1
echo "smoke rc=$?" >> gpurun_out/${T}_smoke.txt
timeout 1500 python -m pytest tests -m "gpu and not slow" -q --timeout 600 > gpurun_out/${T}_pytest.txt 2>&1
echo "pytest rc=$?" >> gpurun_out/${T}_pytest.txt
timeout 1500 python bench.py > gpurun_out/${T}_bench.json 2> gpurun_out/${T}_bench.err
echo "bench rc=$?" >> gpurun_out/${T}_bench.err
timeout 900 python bench.py --impl reference --steps 2 --warmup 1 > gpurun_out/${T}_ref.json 2> gpurun_out/${T}_ref.err
timeout 1200 python tools/bench_apps.py bc c3 16 > gpurun_out/${T}_app_bc_c3.json 2> gpurun_out/${T}_app_bc_c3.err
timeout 900 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv \
  --log-file gpurun_out/${T}_launches_bc_c3.csv python tools/prof_bfs.py --config c3 --reps 1 --app bc --bc-sources 1 > gpurun_out/${T}_launches_bc_c3.log 2>&1
python tools/launches.py gpurun_out/${T}_launches_bc_c3.csv > gpurun_out/${T}_launches_bc_c3.txt 2>&1
timeout 900 python tools/trace_bfs.py c4 2 > gpurun_out/${T}_trace_c4.txt 2>&1
