#!/bin/bash
# full build: GPU parity (new default: pooled flat top-down) + knob sweep
mkdir -p gpurun_out
T=${TAG:-r2s2f}
timeout 300 python -c "import __graft_entry__ as e; e.smoke()" > gpurun_out/${T}_smoke.txt 2>&1
echo "smoke rc=$?" >> gpurun_out/${T}_smoke.txt
timeout 1500 python -m pytest tests -m "gpu and not slow" -x -q --timeout 600 > gpurun_out/${T}_pytest.txt 2>&1
echo "pytest rc=$?" >> gpurun_out/${T}_pytest.txt
TUNES=("" "hub_flat=1" "td_stage=0" "hub_flat=1,td_stage=0" "bu_alpha=20" "bu_alpha=30" "bu_alpha=60" "bu_beta=64" "bu_beta=256")
timeout 900 python tools/sweep_tunes.py c2 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c2.txt 2>&1
timeout 1200 python tools/sweep_tunes.py c4 4 "${TUNES[@]}" > gpurun_out/${T}_sweep_c4.txt 2>&1
timeout 1200 python tools/sweep_tunes.py c3 4 "${TUNES[@]}" > gpurun_out/${T}_sweep_c3.txt 2>&1
