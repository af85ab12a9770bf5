#!/bin/bash
# dev build (K=3): bottom-up kernel at 8 blocks per SM
mkdir -p gpurun_out
T=${TAG:-r2s2aa}
TUNES=("" "bu_minb8=1")
timeout 900 python tools/sweep_tunes.py c2 8 "${TUNES[@]}" > gpurun_out/${T}_sweep_c2.txt 2>&1
timeout 1500 python tools/sweep_tunes.py c4 8 "${TUNES[@]}" > gpurun_out/${T}_sweep_c4.txt 2>&1
timeout 1200 python tools/sweep_tunes.py c3 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c3.txt 2>&1
