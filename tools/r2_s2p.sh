#!/bin/bash
# dev build (K=3): which engine knob slows CC / BC
mkdir -p gpurun_out
T=${TAG:-r2s2p}
TUNES=("" "td_pool=0" "hub_segs=8" "ck_c=32" "td_pool=0,hub_segs=8" "td_pool=0,hub_segs=8,ck_c=32")
timeout 1500 python tools/app_tunes.py bc c3 2 "${TUNES[@]}" > gpurun_out/${T}_bc_c3.txt 2>&1
timeout 900 python tools/app_tunes.py cc c4 3 "${TUNES[@]}" > gpurun_out/${T}_cc_c4.txt 2>&1
timeout 600 python tools/app_tunes.py cc c2 5 "${TUNES[@]}" > gpurun_out/${T}_cc_c2.txt 2>&1
