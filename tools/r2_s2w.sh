#!/bin/bash
# full build: GPU parity (not slow) + BC app timing + BC launch list on C3
mkdir -p gpurun_out
T=${TAG:-r2s2w}
timeout 1500 python -m pytest tests -m "gpu and not slow" -q --timeout 600 > gpurun_out/${T}_pytest.txt 2>&1
echo "pytest rc=$?" >> gpurun_out/${T}_pytest.txt
timeout 1200 python tools/bench_apps.py bc c3 16 > gpurun_out/${T}_app_bc_c3.json 2> gpurun_out/${T}_app_bc_c3.err
timeout 900 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv \
  --log-file gpurun_out/${T}_launches_bc_c3.csv python tools/prof_bfs.py --config c3 --reps 1 --app bc --bc-sources 1 > gpurun_out/${T}_launches_bc_c3.log 2>&1
python tools/launches.py gpurun_out/${T}_launches_bc_c3.csv > gpurun_out/${T}_launches_bc_c3.txt 2>&1
