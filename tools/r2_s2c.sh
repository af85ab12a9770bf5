#!/bin/bash
# dev build (K=3): flat pooled phase B + inline long codewords; sweep td_pool on C2 / C4 / C3
mkdir -p gpurun_out
T=${TAG:-r2s2c}
TUNES=("" "td_pool=1" "td_pool=1,hub_segs=1" "td_stage=0")
timeout 600 python tools/sweep_tunes.py c2 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c2.txt 2>&1
timeout 900 python tools/sweep_tunes.py c4 4 "${TUNES[@]}" > gpurun_out/${T}_sweep_c4.txt 2>&1
timeout 900 python tools/sweep_tunes.py c3 4 "${TUNES[@]}" > gpurun_out/${T}_sweep_c3.txt 2>&1
