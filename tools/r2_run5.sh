#!/bin/bash
mkdir -p gpurun_out
T=${TAG:-r2f}
timeout 150 python tools/dist_debug.py c1 2 > gpurun_out/${T}_distdbg.txt 2>&1
timeout 900 python -m pytest tests/test_gpu_parity.py -m "gpu and not slow" -q --timeout 120 > gpurun_out/${T}_pytest.txt 2>&1
echo "pytest rc=$?" >> gpurun_out/${T}_pytest.txt
timeout 300 python tools/trace_bfs.py c2 2 > gpurun_out/${T}_trace_c2.txt 2>&1
timeout 600 python tools/sweep_tunes.py c2 12 "" "bu_alpha=30" "bu_alpha=35" "bu_alpha=50" > gpurun_out/${T}_sweep_c2.txt 2>&1
timeout 600 python tools/sweep_tunes.py c3 6 "" "bu_alpha=30" "bu_alpha=50" > gpurun_out/${T}_sweep_c3.txt 2>&1
timeout 900 python tools/sweep_tunes.py c4 6 "" "bu_alpha=25" "bu_alpha=30" "bu_alpha=35" > gpurun_out/${T}_sweep_c4.txt 2>&1
timeout 600 python tools/trace_bfs.py c4 1 > gpurun_out/${T}_trace_c4.txt 2>&1
