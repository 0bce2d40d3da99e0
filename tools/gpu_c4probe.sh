cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
for V in "" novote; do for N in 32768 131072 262144 524288 1048576; do
  timeout 120 python tools/c4_probe.py $N $V > gpurun_out/c4p_${N}_$V.log 2>&1; echo "rc=$? $(tail -1 gpurun_out/c4p_${N}_$V.log)"
done; done
