#!/bin/bash
mkdir -p gpurun_out
T=${TAG:-r2g}
timeout 150 python tools/dist_debug.py c1 2 > gpurun_out/${T}_distdbg.txt 2>&1
timeout 400 python -m pytest tests/test_dist.py -m "gpu" -q --timeout 150 > gpurun_out/${T}_pytest_dist.txt 2>&1
echo "pytest rc=$?" >> gpurun_out/${T}_pytest_dist.txt
timeout 900 python -m pytest tests/test_gpu_parity.py -m "gpu and not slow" -q --timeout 120 > gpurun_out/${T}_pytest.txt 2>&1
echo "pytest rc=$?" >> gpurun_out/${T}_pytest.txt
timeout 300 python tools/trace_bfs.py c3 1 > gpurun_out/${T}_trace_c3.txt 2>&1
timeout 600 python tools/sweep_tunes.py c2 12 "" "bu_alpha=20" "bu_alpha=25" "td_pool=1" "td_pool=1,bu_alpha=25" > gpurun_out/${T}_sweep_c2.txt 2>&1
timeout 600 python tools/sweep_tunes.py c3 8 "" "bu_alpha=20" "bu_alpha=25" "bu_hub_segs=100000" "hub_segs=2" "td_pool=1" > gpurun_out/${T}_sweep_c3.txt 2>&1
timeout 900 python tools/sweep_tunes.py c4 8 "bu_alpha=25" "bu_alpha=20" "bu_alpha=25,td_pool=1" "bu_alpha=25,bu_hub_segs=100000" > gpurun_out/${T}_sweep_c4.txt 2>&1
