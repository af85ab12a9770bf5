#!/bin/bash
# dev build (K=3): checkpoint chunk size (long interval areas grid-wide) and deferred bottom-up hubs (flat pass)
mkdir -p gpurun_out
T=${TAG:-r2s2j}
TUNES=("" "ck_c=16" "ck_c=8" "ck_c=4" "bu_hub_segs=1" "bu_hub_segs=2" "bu_hub_segs=4" "bu_hub_segs=2,bu_hub_flat=0")
timeout 900 python tools/sweep_tunes.py c2 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c2.txt 2>&1
timeout 1200 python tools/sweep_tunes.py c4 4 "${TUNES[@]}" > gpurun_out/${T}_sweep_c4.txt 2>&1
timeout 1200 python tools/sweep_tunes.py c3 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c3.txt 2>&1
