cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
O=gpurun_out/diag6.log; : > $O
rm -f /tmp/diag.pid
cat > /tmp/gdbcmds <<'G'
set pagination off
set cuda break_on_launch none
run
info cuda kernels
info cuda sms
info cuda warps
bt
x/8i $pc
cuda sm 1
info cuda warps
cuda sm 60
info cuda warps
cuda sm 120
info cuda warps
info cuda lanes
bt
x/6i $pc
kill
quit
G
DIAG_PIDFILE=/tmp/diag.pid DIAG_TIMEOUT=600 timeout 400 /usr/local/cuda/bin/cuda-gdb -batch -x /tmp/gdbcmds --args python tools/split_diag.py C5 0 20 > $O 2>&1 &
G=$!
for i in $(seq 1 60); do [ -f /tmp/diag.pid ] && break; sleep 1; done
sleep 40
kill -INT $(cat /tmp/diag.pid)
wait $G
grep -v "^\[New Thread\|Thread .* exited\|libthread_db" $O | head -400 > gpurun_out/diag6_short.log
