#!/bin/bash
# full build: GPU parity (not slow) + BC / BFS / CC app timings
mkdir -p gpurun_out
T=${TAG:-r2s2u}
timeout 1500 python -m pytest tests -m "gpu and not slow" -q --timeout 600 > gpurun_out/${T}_pytest.txt 2>&1
echo "pytest rc=$?" >> gpurun_out/${T}_pytest.txt
timeout 1200 python tools/bench_apps.py bc c3 8 > gpurun_out/${T}_app_bc_c3.json 2> gpurun_out/${T}_app_bc_c3.err
timeout 900 python tools/bench_apps.py bfs c3 8 > gpurun_out/${T}_app_bfs_c3.json 2> gpurun_out/${T}_app_bfs_c3.err
timeout 900 python tools/bench_apps.py bfs c2 8 > gpurun_out/${T}_app_bfs_c2.json 2> gpurun_out/${T}_app_bfs_c2.err
timeout 900 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv \
  --log-file gpurun_out/${T}_launches_bc_c3.csv python tools/prof_bfs.py --config c3 --reps 1 --app bc --bc-sources 1 > gpurun_out/${T}_launches_bc_c3.log 2>&1
python tools/launches.py gpurun_out/${T}_launches_bc_c3.csv > gpurun_out/${T}_launches_bc_c3.txt 2>&1
