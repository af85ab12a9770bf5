#!/bin/bash
mkdir -p gpurun_out
T=${TAG:-r2k}
timeout 900 python -m pytest tests/test_gpu_parity.py -m "gpu and not slow" -q --timeout 120 > gpurun_out/${T}_pytest.txt 2>&1
echo "pytest rc=$?" >> gpurun_out/${T}_pytest.txt
TUNES=("ck_c=0,bu_grow=0,bu_alpha=25" "bu_grow=0,bu_alpha=25" "bu_grow=0,bu_alpha=30" "bu_alpha=40" "bu_alpha=50" "ck_c=64,bu_grow=0,bu_alpha=25")
timeout 600 python tools/sweep_tunes.py c2 8 "${TUNES[@]}" > gpurun_out/${T}_sweep_c2.txt 2>&1
timeout 800 python tools/sweep_tunes.py c3 8 "${TUNES[@]}" > gpurun_out/${T}_sweep_c3.txt 2>&1
timeout 1000 python tools/sweep_tunes.py c4 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c4.txt 2>&1
