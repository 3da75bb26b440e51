#!/bin/bash
# compute-sanitizer racecheck + synccheck (+ memcheck) over every hot-path kernel at small sizes:
# the one-pass kernels (streamed-residual rl, gathered-residual rg, general), the select tile kernel
# and compaction (one tile per CTA and the persistent tile-buffer mode), the ordered refine, refine+SUM,
# SUM, MIN/MAX, grouping; split residuals (streamed high planes, host check entries).  Summaries go to
# gpurun_out/sanitize_*.txt.  CFGS="name:ENV=V,ENV=V name2:..." restricts the configurations.
out=gpurun_out
for tool in racecheck synccheck memcheck; do
  for cfg in ${CFGS:-"base:" "rg:AR_RL_RESMODE=2" "host:RES_LOC=1" "legacy:AR_FUSED_LEGACY=1" "seltile:AR_SEL_RR=0" "selbufs:AR_SEL_RR=0,AR_SEL_BUFS=2" "selrr3:AR_SEL_RR_GRID=3" "split:SPLIT=4" "splithost:SPLIT=4 RES_LOC=1" "split3host:SPLIT=3 RES_LOC=1"}; do
    name=${cfg%%:*}; envs=${cfg#*:}; envs=${envs//,/ }
    extra=""
    [ "$tool" = "racecheck" ] && extra="--racecheck-report all"
    env $envs N=${N:-70001} timeout 1200 compute-sanitizer --tool $tool $extra --print-limit 50 \
        python tools/sanitize_driver.py > $out/sanitize_${tool}_${name}.txt 2>&1
    echo "$tool $name rc=$? $(grep -E 'ERROR SUMMARY|RACECHECK SUMMARY|sanitize driver ok' $out/sanitize_${tool}_${name}.txt | tr '\n' ' ')"
  done
done
