# session-4 direction-threshold sweep (run under gpurun): bu_beta / bu_alpha / bu on C2 (web) and C3 (social)
mkdir -p gpurun_out
T="bu_beta=24 bu_beta=32 bu_beta=48 bu_beta=64 bu_beta=96 bu_beta=128 bu_beta=256 bu_beta=64,bu=2 bu_beta=64,bu_alpha=5"
timeout 600 python tools/sweep.py c2 $T > gpurun_out/sw2_c2.txt 2>&1
timeout 600 python tools/sweep.py c3 $T > gpurun_out/sw2_c3.txt 2>&1
cat gpurun_out/sw2_c2.txt gpurun_out/sw2_c3.txt
