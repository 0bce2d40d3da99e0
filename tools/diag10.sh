cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
O=gpurun_out/diag10.log; : > $O
run() { echo "== $*" >> $O; timeout 100 env "$@" >> $O 2>&1 || echo "rc=$?" >> $O; }
run CULI_SPLIT_STATS=1 DIAG_TIMEOUT=60 python tools/split_diag.py C2 0 1
run CULI_SPLIT_STATS=1 DIAG_TIMEOUT=60 CULI_STEAL_GATE=0 python tools/split_diag.py C2 0 1
grep "^C\|^==\|rc=\|culi split" $O
