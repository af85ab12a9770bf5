#!/bin/bash
# full build: vertex-rule threshold with the growth-guarded edge test
mkdir -p gpurun_out
T=${TAG:-r2s2v}
TUNES=("" "bu_alpha=35" "bu_alpha=30" "bu_alpha=25" "bu_alpha=30,bu_grow=0" "nfilter=1")
timeout 900 python tools/sweep_tunes.py c2 8 "${TUNES[@]}" > gpurun_out/${T}_sweep_c2.txt 2>&1
timeout 1500 python tools/sweep_tunes.py c4 8 "${TUNES[@]}" > gpurun_out/${T}_sweep_c4.txt 2>&1
timeout 1200 python tools/sweep_tunes.py c3 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c3.txt 2>&1
